"""Pipe utilisation of one kernel from an `ncu --set full` report, stored under a tag in
profiles/prune_pipe.json (bench.py reports it beside the roofline fraction) and
profiles/prune_traffic.json (DRAM bytes per launch).

usage: python tools/ncu_pipe_json.py REPORT.ncu-rep TAG PARTIALS_PER_LAUNCH [source note]

FP instructions executed per launch = the sum over SM sub-partitions of the
per-cycle thread-instruction rates (DFMA + DMUL + DADD, or FFMA + FMUL + FADD)
times the elapsed SM cycles; divided by the algorithmic site-node partials of the
launch this gives the FP instructions the kernel really issues per partial (the
metric's 21.8 flops per partial count what the method needs, the tables skip some)."""
import csv
import json
import os
import subprocess
import sys

rep, tag, partials = sys.argv[1], sys.argv[2], float(sys.argv[3])
note = sys.argv[4] if len(sys.argv) > 4 else rep
out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
r = list(csv.reader(out.splitlines()))
d = dict(zip(r[0], r[2]))
units = dict(zip(r[0], r[1]))
SCALE = {"byte": 1.0, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "KB": 1e3, "MB": 1e6, "GB": 1e9}


def nbytes(k):
    return f(k) * SCALE.get(units.get(k, "byte"), 1.0)


def f(k):
    try:
        return float(d[k])
    except (KeyError, ValueError):
        return 0.0


cyc = f("sm__cycles_elapsed.avg")
rate = lambda ops: sum(f(f"smsp__sass_thread_inst_executed_op_{o}_pred_on.sum.per_cycle_elapsed") for o in ops)
fp64 = rate(["dfma", "dmul", "dadd"]) * cyc
fp32 = rate(["ffma", "fmul", "fadd"]) * cyc
ms = f("gpu__time_duration.sum")
entry = {
    "kernel": r[2][r[0].index("Kernel Name")] if "Kernel Name" in r[0] else None,
    "ncu_duration_ms": ms,
    "fp64_pipe_active_pct": f("sm__pipe_fp64_cycles_active.avg.pct_of_peak_sustained_active"),
    "fma_pipe_active_pct": f("sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active"),
    "issue_active_pct": f("smsp__issue_active.avg.pct_of_peak_sustained_active"),
    "warps_active_pct": f("sm__warps_active.avg.pct_of_peak_sustained_active"),
    "registers": f("launch__registers_per_thread"),
    "warp_inst_per_launch": f("smsp__inst_executed.sum"),
    "fp64_thread_inst_per_partial": fp64 / partials if fp64 else None,
    "fp32_thread_inst_per_partial": fp32 / partials if fp32 else None,
    "shared_bank_conflicts": f("l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum"),
    "shared_wavefronts": f("l1tex__data_pipe_lsu_wavefronts_mem_shared.sum"),
    # one shared-memory wavefront per SM per cycle at most
    "shared_wavefront_pct": 100.0 * f("l1tex__data_pipe_lsu_wavefronts_mem_shared.sum") /
                            max(1.0, f("sm__cycles_elapsed.avg") * f("device__attribute_multiprocessor_count")),
    "dram_bytes": nbytes("dram__bytes_read.sum") + nbytes("dram__bytes_write.sum"),
    "source": note,
}
root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
for name, val in (("prune_pipe.json", entry), ("prune_traffic.json", entry["dram_bytes"])):
    p = os.path.join(root, "profiles", name)
    try:
        js = json.load(open(p))
    except Exception:
        js = {}
    js[tag] = val
    json.dump(js, open(p, "w"), indent=1, sort_keys=True)
print(json.dumps(entry, indent=1))
