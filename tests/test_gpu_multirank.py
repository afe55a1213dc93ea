"""World-size invariance on one GPU: P virtual ranks, each a
context with (rank, world = P) scoring only its slots, exchange records
through the C ABI (mpcgs_get_records / mpcgs_put_records) and draw with
mpcgs_step_finish.  Every rank must reproduce the world = 1 chain bit for bit:
same records, same draws, same generator.  Each rank tiles its pruning launch
for its own N/P proposals (rank-local tiling); the site sums are exact
(arith.cuh Exact128), so the records still agree bitwise.  The 20 kbp cases
make the tilings differ (checked through the tiling the library reports)."""
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


@pytest.mark.parametrize("world", [2, 4, 8])
@pytest.mark.parametrize("precision,L,incremental", [(64, 700, False), (32, 700, False), (64, 20000, False),
                                                     (32, 20000, False), (64, 20000, True)])
def test_virtual_ranks_reproduce_single_gpu_chain(P, world, precision, L, incremental):
    wl = synth.workload("c2", L=L)
    rows = synth.to_strings(wl["codes"])
    N, K, seed, steps = 64, 64, wl["chain_seed"], 8
    tree = (wl["true_parent"], wl["true_age"])
    kw = dict(init_tree=tree, precision=precision, max_proposals=N, max_samples=4, incremental=incremental)
    ref = P.Context(rows, wl["theta0"], **kw)
    ranks = [P.Context(rows, wl["theta0"], rank=r, world=world, **kw) for r in range(world)]
    if L == 20000 and not incremental:  # the rank-local tilings really differ from world = 1
        assert P.mpcgs_prune_tiling(12, L, N, precision) != P.mpcgs_prune_tiling(12, L, N // world, precision)
    for step in range(steps):
        tr = ref.mpcgs_step_trace(step, N, K, seed)
        for c in ranks:
            c.mpcgs_step_local(step, N, seed)
        full = np.concatenate([c.mpcgs_get_records(*P.mpcgs_shard_range(N, r, world)) for r, c in enumerate(ranks)])
        assert np.array_equal(full[:, 0], tr["logL"][1:])   # bitwise: same kernels, same tiling
        assert np.array_equal(full[:, 1], tr["S"][1:])
        for c in ranks:
            c.mpcgs_put_records(1, full)
        for c in ranks:
            assert np.array_equal(c.mpcgs_step_finish(step, N, K, seed), tr["draws"])
        gp, ga, gl, gS = ref.mpcgs_get_state()
        for c in ranks:
            p2, a2, l2, S2 = c.mpcgs_get_state()
            assert np.array_equal(p2, gp) and np.array_equal(a2, ga) and l2 == gl and S2 == gS


def test_sample_refuses_world_gt1_without_nccl(P):
    wl = synth.workload("c1")
    c = P.Context(synth.to_strings(wl["codes"]), wl["theta0"], max_proposals=16, max_samples=16, rank=0, world=2)
    with pytest.raises(P.MpcgsError) as ei:
        c.mpcgs_sample(16, 16, 1)
    assert ei.value.status == -3


def test_nccl_path_single_rank_matches(P):
    """The in-library NCCL all-gather path (dlopen'ed NCCL, communicator from an
    ncclUniqueId, all-gather inside the captured step loop) with one rank gives
    the same chain as the communicator-free path."""
    wl = synth.workload("c2", L=500)
    rows = synth.to_strings(wl["codes"])
    tree = (wl["true_parent"], wl["true_age"])
    a = P.Context(rows, wl["theta0"], init_tree=tree, max_proposals=64, max_samples=640, burnin_steps=3)
    uid = P.mpcgs_nccl_unique_id()
    assert len(uid) == 128
    b = P.Context(rows, wl["theta0"], init_tree=tree, max_proposals=64, max_samples=640, burnin_steps=3,
                  nccl_id=uid)
    for c in (a, b):
        c.mpcgs_sample(64, 640, 5)
    sa, sb = a.mpcgs_get_samples(), b.mpcgs_get_samples()
    for k in sa:
        assert np.array_equal(sa[k], sb[k]), k


def test_nccl_two_ranks_match_single_gpu():
    """P22 over a real NCCL communicator: 2 processes (torchrun), each scoring half
    of the proposals and all-gathering the records inside mpcgs_sample's captured
    loop, reproduce the 1-GPU samples bit for bit.  Needs 2 GPUs (skipped below)."""
    import os
    import subprocess
    import sys

    import torch

    if torch.cuda.device_count() < 2:
        pytest.skip("needs 2 GPUs")
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    r = subprocess.run([sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node=2",
                        "--master-addr", "127.0.0.1", "--master-port", "29533",
                        os.path.join(root, "tools", "nccl_check.py")], capture_output=True, text=True, timeout=900)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    assert "identical" in r.stdout
