"""bench.py end to end on a small workload (the driver's contract: one JSON line with
metric, value, roofline, cpu_baseline, e2e, clocks, gpu_launches), and the reference
arm on the CPU oracle."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _run(*args, timeout=600):
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], capture_output=True, text=True,
                       timeout=timeout, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    return json.loads(r.stdout.strip().splitlines()[-1])


@pytest.mark.gpu
def test_bench_line_contract():
    d = _run("--workload", "c2", "--steps", "4", "--warmup", "3", "--cpu-seconds", "2")
    for k in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better", "dtype",
              "config", "roofline", "cpu_baseline", "e2e", "gpu_launches", "clocks", "theta_mle",
              "phases_ms_per_step", "production_loop"):
        assert k in d, k
    assert d["value"] > 0 and d["gpu_launches"] > 0
    r = d["roofline"]
    assert r["bound"] == "alu" and 0 < r["frac"] < 1.5 and r["peak"] > 1
    assert d["e2e"]["value"] > 0 and d["e2e"]["h2d_bytes_per_step"] > 0
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] >= 1


def test_bench_reference_arm_cpu():
    d = _run("--impl", "reference", "--workload", "c1", "--steps", "2", "--warmup", "1", timeout=300)
    assert d["impl"] == "reference" and d["value"] > 0
    assert d["e2e"]["h2d_bytes_per_step"] == 0 and d["cpu_baseline"]["kind"] == "oracle"


@pytest.mark.gpu
@pytest.mark.parametrize("extra", [["--ambiguity", "0.05"], ["--model", "F84", "--kappa", "2.0"],
                                   ["--precision", "32", "--incremental"]])
def test_bench_variant_lines(extra):
    """The optional workload switches each produce a valid line."""
    d = _run("--workload", "c2", "--steps", "3", "--warmup", "3", "--cpu-seconds", "1", *extra)
    assert d["value"] > 0 and d["gpu_launches"] > 0
    if "--incremental" in extra:  # no flop-count fraction for incremental rescoring (bench.py)
        assert d["roofline"]["kernel"] == "k_score_incr" and d["roofline"]["frac"] is None
    else:
        assert d["roofline"]["frac"] > 0
