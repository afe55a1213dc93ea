"""Multi-process plumbing for proposal sharding.

One process per GPU.  Rank r owns proposal slots mpcgs_shard_range(N, r, P);
every rank holds the replicated generator, so after each rank has scored its
slots the only exchange is the per-slot records (5 doubles: lnL, S, t1, t2,
pair).  Two ways to do it:

* in the library: rank 0 makes an ncclUniqueId (``broadcast_nccl_id``), every
  rank passes it to ``Context(..., nccl_id=...)``, and ``mpcgs_sample`` runs an
  in-place ncclAllGather of the records inside its device step loop;
* host-staged (any torch.distributed backend, e.g. gloo): ``sharded_step``
  drives ``mpcgs_step_local`` -> ``mpcgs_get_records`` -> ``exchange_records``
  -> ``mpcgs_put_records`` -> ``mpcgs_step_finish``.

Both give the same chain as one GPU (world-size invariance, P22) because
every random number is a Philox counter of (seed, step, slot) and the pruning
tiling depends only on the global N.
"""
from __future__ import annotations

import numpy as np

from .mpcgs import REC, mpcgs_nccl_unique_id, mpcgs_shard_range


def broadcast_nccl_id(group=None, device=None, make_id=mpcgs_nccl_unique_id) -> bytes:
    """Rank 0 creates a 128-byte id; every rank returns the same bytes."""
    import torch
    import torch.distributed as dist

    buf = torch.zeros(128, dtype=torch.uint8, device=device or "cpu")
    if dist.get_rank(group) == 0:
        buf.copy_(torch.frombuffer(bytearray(make_id()), dtype=torch.uint8))
    dist.broadcast(buf, src=0, group=group)
    return bytes(buf.cpu().numpy().tobytes())


def exchange_records(local: np.ndarray, n_proposals: int, group=None) -> np.ndarray:
    """All-gather each rank's [count, 5] records into the [N, 5] records of
    slots 1..N (rank order == slot order, mpcgs_shard_range)."""
    import torch
    import torch.distributed as dist

    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    first, count = mpcgs_shard_range(n_proposals, rank, world)
    local = np.ascontiguousarray(local, dtype=np.float64).reshape(count, REC)
    out = torch.empty(world * count * REC, dtype=torch.float64)
    dist.all_gather_into_tensor(out, torch.from_numpy(local.reshape(-1).copy()), group=group)
    full = out.numpy().reshape(n_proposals, REC)
    assert first == 1 + rank * count
    return full


def sharded_step(ctx, step: int, n_proposals: int, n_draws: int, seed: int, group=None) -> np.ndarray:
    """One GMH step with host-staged record exchange; returns the draw indices."""
    import torch.distributed as dist

    rank, world = dist.get_rank(group), dist.get_world_size(group)
    first, count = mpcgs_shard_range(n_proposals, rank, world)
    ctx.mpcgs_step_local(step, n_proposals, seed)
    rec = ctx.mpcgs_get_records(first, count)
    full = exchange_records(rec, n_proposals, group)
    ctx.mpcgs_put_records(1, full)
    return ctx.mpcgs_step_finish(step, n_proposals, n_draws, seed)
