"""P22 over NCCL (run under torchrun, one process per GPU): every rank samples a
c2-shaped chain with the proposals sharded over the world and the records
all-gathered by the library's in-graph ncclAllGather; rank 0 also samples the
same chain alone (world = 1, its own context) and compares the sample stores and
final genealogies bit for bit.  Prints "identical" and exits 0 on success."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402

import synth  # noqa: E402
import paper_conf_ipps_davistzw17_b200 as P  # noqa: E402
from paper_conf_ipps_davistzw17_b200 import dist as D  # noqa: E402


def main():
    rank, world = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    local = int(os.environ.get("LOCAL_RANK", rank))
    torch.cuda.set_device(local)
    dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    ok = True
    for L, N, M in ((700, 64, 6400), (20000, 64, 1280)):
        wl = synth.workload("c2", L=L)
        rows = synth.to_strings(wl["codes"])
        kw = dict(init_tree=(wl["true_parent"], wl["true_age"]), max_proposals=N, max_samples=M, burnin_steps=5)
        uid = D.broadcast_nccl_id(device=torch.device("cuda", local))
        ctx = P.Context(rows, wl["theta0"], rank=rank, world=world, nccl_id=uid, **kw)
        ctx.mpcgs_sample(N, M, wl["chain_seed"])
        got = ctx.mpcgs_get_samples()
        gen = ctx.mpcgs_get_state()
        if rank == 0:
            one = P.Context(rows, wl["theta0"], **kw)
            one.mpcgs_sample(N, M, wl["chain_seed"])
            ref = one.mpcgs_get_samples()
            same = all(np.array_equal(got[k], ref[k]) for k in ref)
            g1 = one.mpcgs_get_state()
            same = same and np.array_equal(gen[0], g1[0]) and np.array_equal(gen[1], g1[1]) and gen[2] == g1[2]
            print(f"L={L} world={world}: {'identical' if same else 'DIFFERENT'}", flush=True)
            ok = ok and same
    flag = torch.tensor([1 if ok else 0], device="cuda")
    dist.all_reduce(flag, op=dist.ReduceOp.MIN)
    dist.destroy_process_group()
    if rank == 0 and ok:
        print("identical")
    return 0 if int(flag.item()) else 1


if __name__ == "__main__":
    sys.exit(main())
