"""World-size invariance (P22) under the current tiling policy (MPCGS_TILING_WORLD
in the environment): P virtual ranks must reproduce the world = 1 chain bit for
bit.  Exit status 0 = identical.  Used by tests/test_gpu_multirank.py in a
subprocess (the policy is read once per process)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402

import synth  # noqa: E402
import paper_conf_ipps_davistzw17_b200 as P  # noqa: E402


def main(world=8, L=20000, N=64, steps=3):
    wl = synth.workload("c2", L=L)
    rows = synth.to_strings(wl["codes"])
    seed, tree = wl["chain_seed"], (wl["true_parent"], wl["true_age"])
    ref = P.Context(rows, wl["theta0"], init_tree=tree, max_proposals=N, max_samples=4)
    ranks = [P.Context(rows, wl["theta0"], init_tree=tree, max_proposals=N, max_samples=4, rank=r, world=world)
             for r in range(world)]
    for step in range(steps):
        tr = ref.mpcgs_step_trace(step, N, N, seed)
        for c in ranks:
            c.mpcgs_step_local(step, N, seed)
        full = np.concatenate([c.mpcgs_get_records(*P.mpcgs_shard_range(N, r, world)) for r, c in enumerate(ranks)])
        if not np.array_equal(full[:, 0], tr["logL"][1:]):
            print("logL differ at step", step)
            return 1
        for c in ranks:
            c.mpcgs_put_records(1, full)
        for c in ranks:
            if not np.array_equal(c.mpcgs_step_finish(step, N, N, seed), tr["draws"]):
                print("draws differ at step", step)
                return 1
    print("identical", os.environ.get("MPCGS_TILING_WORLD", "1"))
    return 0


if __name__ == "__main__":
    sys.exit(main(*(int(a) for a in sys.argv[1:])))
