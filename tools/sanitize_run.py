"""Small end-to-end run touching every kernel, for compute-sanitizer
(memcheck / racecheck / synccheck) on the GPU box."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402

import synth  # noqa: E402
import paper_conf_ipps_davistzw17_b200 as P  # noqa: E402

for prec in (64, 32):
    for inc in (False, True):
        for name, over in (("c1", {}), ("c4", {"n": 128, "L": 300, "N": 16})):
            wl = synth.workload(name, **over)
            rows = synth.to_strings(wl["codes"])
            N = wl["N"]
            c = P.Context(rows, wl["theta0"], precision=prec, incremental=inc, burnin_steps=2, max_proposals=N,
                          max_samples=4 * N)
            c.mpcgs_step_trace(0, N, N, 7)
            c.mpcgs_sample(N, 4 * N, 3)
            th = c.mpcgs_estimate_theta(32)
            p, a, _, _ = c.mpcgs_get_state()
            c.mpcgs_score_trees(np.stack([p, wl["true_parent"]]), np.stack([a, wl["true_age"]]))
            c.free()
            print(name, prec, inc, "theta-hat", th)
print("sanitize run done")
