"""Parity at BASELINE.json's full sizes, in the launch configuration bench.py
times (one GMH step through mpcgs_step_trace with all N proposals), checked
on outputs the oracle can compute one by one: the target, every proposal's
resimulated times / pair code / S_G, the likelihood of a sample of proposals
(full-alignment oracle pruning), and the draws from the GPU likelihoods
(inverse CDF recomputed on the host from the same weights)."""
import os
from concurrent.futures import ThreadPoolExecutor

import numpy as np
import pytest

import synth

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def P():
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_ipps_davistzw17_b200 as pkg

    pkg.lib()
    return pkg


CASES = [
    ("c3", {}, 32),                 # 24 x 1,000 bp, N = 256
    ("c4", {"n": 256}, 32),         # 256 x 2,000 bp, N = 512 (largest n of the sweep)
    ("c5", {}, 64),                 # 64 x 100,000 bp, N = 1,024 (the bench workload)
]


@pytest.mark.parametrize("precision,incremental", [(64, False), (32, False), (64, True)])
@pytest.mark.parametrize("name,over,n_ll", CASES)
def test_full_size_step_sampled_parity(P, orc, name, over, n_ll, precision, incremental):
    if (precision, incremental) != (64, False) and name != "c5":
        pytest.skip("FP32 and incremental rescoring are checked at the bench workload")
    wl = synth.workload(name, **over)
    codes = wl["codes"]
    n, L = codes.shape
    N = wl["N"]
    pi = orc.base_freqs(codes)
    u = orc.default_rate(pi)
    theta0 = wl["theta0"]
    parent, age = wl["true_parent"], wl["true_age"]
    ctx = P.Context(synth.to_strings(codes), theta0, init_tree=(parent, age), max_proposals=N, max_samples=16,
                    precision=precision, incremental=incremental)
    tol = 1e-9 if precision == 64 else 1e-4
    seed, step = wl["chain_seed"], 3
    tr = ctx.mpcgs_step_trace(step, N, N, seed)
    assert tr["target"] == orc.pick_target(parent, seed, step)
    scale = age.max()
    rng = np.random.default_rng(0)
    ll_slots = set(rng.choice(np.arange(1, N + 1), size=n_ll, replace=False).tolist())
    flagged = 0
    ll_trees = []
    for slot in range(1, N + 1):
        p2, a2, t12, pair, flag = orc.propose(parent, age, theta0, tr["target"], seed, step, slot)
        if flag:
            flagged += 1
            continue
        assert tr["pair"][slot] == pair, slot
        assert np.allclose(tr["t12"][slot], t12, rtol=0, atol=1e-12 * max(scale, t12[1]))
        assert abs(tr["S"][slot] - orc.coalescent_S(a2, n)) <= 1e-12 * abs(tr["S"][slot])
        if slot in ll_slots:
            ll_trees.append((slot, p2, a2))
    assert flagged <= 2
    # the sampled proposals' full-alignment oracle likelihoods, on the host's cores (the
    # oracle is a C library called through ctypes, which releases the GIL)
    with ThreadPoolExecutor(max_workers=min(len(ll_trees), os.cpu_count() or 1) or 1) as ex:
        wants = list(ex.map(lambda t: orc.log_likelihood(codes, t[1], t[2], pi, u), ll_trees))
    for (slot, _, _), want in zip(ll_trees, wants):
        assert abs(tr["logL"][slot] - want) <= tol * abs(want), (slot, tr["logL"][slot], want)
    if precision == 32:  # FP32 gets logL tolerance, not index parity (P21)
        return
    # draws: inverse CDF over softmax of the GPU likelihoods, lowest index on ties
    w, cum = orc.weights(tr["logL"])
    for d, got in enumerate(tr["draws"]):
        i, near = orc.draw(cum, orc.uniform(seed, 0, step, orc.TAG_DRAW, d))
        if not near:
            assert got == i
