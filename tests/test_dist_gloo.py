"""World-size-2 gloo test (CPU) of the proposal-sharding host logic
(SURVEY 8(e), P22): slot partition, id broadcast and the record exchange of
paper_conf_ipps_davistzw17_b200.dist.  Each rank computes the records of its
own slots (the oracle stands in for the per-rank GPU work, which needs a
device); after the all-gather both ranks must hold exactly the records and
draws of the single-process oracle step."""
import os
import socket
import sys

import numpy as np
import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def _worker(rank, world, port, steps, q):
    sys.path.insert(0, ROOT)
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    import torch.distributed as dist

    import oracle as orc
    import synth
    from paper_conf_ipps_davistzw17_b200 import dist as D
    from paper_conf_ipps_davistzw17_b200 import mpcgs_shard_range

    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        idb = D.broadcast_nccl_id(make_id=lambda: bytes(range(128)))
        assert idb == bytes(range(128))
        wl = synth.workload("c1")
        codes = wl["codes"]
        n = codes.shape[0]
        pi = orc.base_freqs(codes)
        u = orc.default_rate(pi)
        theta0 = wl["theta0"]
        parent, age = orc.upgma(codes, theta0)
        gl = orc.log_likelihood(codes, parent, age, pi, u)
        N, K, seed = 16, 16, wl["chain_seed"]
        first, count = mpcgs_shard_range(N, rank, world)
        for step in range(steps):
            target = orc.pick_target(parent, seed, step)
            local = []
            for slot in range(first, first + count):
                p2, a2, t12, pair, _ = orc.propose(parent, age, theta0, target, seed, step, slot)
                local.append([orc.log_likelihood(codes, p2, a2, pi, u), orc.coalescent_S(a2, n), t12[0], t12[1], pair])
            full = D.exchange_records(np.array(local), N)
            ref = orc.gmh_step(codes, pi, u, theta0, N, K, seed, step, parent, age, gl)
            assert np.array_equal(full[:, 0], ref["logL"][1:])
            assert np.array_equal(full[:, 1], ref["S"][1:])
            assert np.array_equal(full[:, 2:4], ref["t12"][1:])
            assert np.array_equal(full[:, 4].astype(int), ref["pair"][1:])
            _, cum = orc.weights(np.concatenate([[gl], full[:, 0]]))
            draws = [orc.draw(cum, orc.uniform(seed, 0, step, orc.TAG_DRAW, d))[0] for d in range(K)]
            assert draws == list(ref["draws"])
            parent, age, gl = ref["parent"], ref["age"], ref["gen_logL"]
        q.put((rank, "ok"))
    except Exception as e:  # report to the parent
        q.put((rank, repr(e)))
    finally:
        dist.destroy_process_group()


def test_gloo_world2_sharded_step_equals_single_process():
    import torch.multiprocessing as mp

    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, 6, q)) for r in range(2)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=240) for _ in procs)
    for p in procs:
        p.join(timeout=60)
    assert res == {0: "ok", 1: "ok"}, res
