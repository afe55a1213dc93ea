"""Two processes, one GPU: each process is a rank with its own
context (rank, world = 2) scoring only its proposal slots on cuda:0, and the record
exchange goes through torch.distributed (gloo) with paper_conf_ipps_davistzw17_b200.dist
-- the real multi-process plumbing of proposal sharding (dist.sharded_step), with the
per-rank GPU work the CPU gloo test can only stand in for.  Both ranks must reproduce the
single-process chain bit for bit (draws, generator, likelihoods)."""
import os
import socket
import sys

import numpy as np
import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
pytestmark = pytest.mark.gpu


def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def _worker(rank, world, port, steps, q):
    sys.path.insert(0, ROOT)
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    import torch
    import torch.distributed as dist

    import synth
    import paper_conf_ipps_davistzw17_b200 as P
    from paper_conf_ipps_davistzw17_b200 import dist as D

    torch.cuda.set_device(0)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        wl = synth.workload("c2", L=3000)
        rows = synth.to_strings(wl["codes"])
        N, seed = 64, wl["chain_seed"]
        tree = (wl["true_parent"], wl["true_age"])
        ctx = P.Context(rows, wl["theta0"], init_tree=tree, max_proposals=N, max_samples=4, rank=rank, world=world)
        ref = P.Context(rows, wl["theta0"], init_tree=tree, max_proposals=N, max_samples=4) if rank == 0 else None
        for step in range(steps):
            draws = D.sharded_step(ctx, step, N, N, seed)
            if ref is not None:
                tr = ref.mpcgs_step_trace(step, N, N, seed)
                assert np.array_equal(draws, tr["draws"]), step
                first, count = P.mpcgs_shard_range(N, 0, world)
                assert np.array_equal(ctx.mpcgs_get_records(first, count)[:, 0], tr["logL"][first:first + count])
                g1, g2 = ctx.mpcgs_get_state(), ref.mpcgs_get_state()
                assert np.array_equal(g1[0], g2[0]) and np.array_equal(g1[1], g2[1]) and g1[2] == g2[2]
        # both ranks hold the same generator
        p, a, ll, S = ctx.mpcgs_get_state()
        buf = torch.tensor(np.concatenate([a, [ll, S]]), dtype=torch.float64)
        out = [torch.zeros_like(buf) for _ in range(world)]
        dist.all_gather(out, buf)
        assert all(torch.equal(out[0], o) for o in out)
        q.put((rank, "ok"))
    except Exception as e:  # report to the parent
        import traceback

        q.put((rank, repr(e) + traceback.format_exc()[-1500:]))
    finally:
        dist.destroy_process_group()


def test_two_processes_one_gpu_match_single_process():
    import torch
    import torch.multiprocessing as mp

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, 6, q)) for r in range(2)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=600) for _ in procs)
    for p in procs:
        p.join(timeout=120)
    assert res == {0: "ok", 1: "ok"}, res
