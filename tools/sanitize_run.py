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
        for name, over in (("c1", {}), ("c3", {"L": 600, "N": 32}), ("c4", {"n": 128, "L": 300, "N": 16})):
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
# compressed patterns, virtual ranks (records through the host), loaded samples (a7)
wl = synth.workload("c2", L=700)
rows = synth.to_strings(wl["codes"])
c = P.Context(rows, wl["theta0"], compress_patterns=True, max_proposals=64, max_samples=256)
c.mpcgs_sample(64, 256, 5)
r = [P.Context(rows, wl["theta0"], max_proposals=64, max_samples=4, rank=k, world=2) for k in range(2)]
for k, ck in enumerate(r):
    ck.mpcgs_step_local(0, 64, 9)
full = np.concatenate([ck.mpcgs_get_records(*P.mpcgs_shard_range(64, k, 2)) for k, ck in enumerate(r)])
for ck in r:
    ck.mpcgs_put_records(1, full)
    ck.mpcgs_step_finish(0, 64, 64, 9)
c.mpcgs_load_samples(np.array([1.0, 100.0, 3.0]), 2.15)
print("bimodal theta-hat", c.mpcgs_estimate_theta(64))
# n = 256 (single code buffer, setup arrays aliased into the spill levels), F81 and HKY85
for model, kappa in (("F81", 0.0), ("HKY85", 4.0)):
    wl = synth.workload("c4", n=256, L=600, N=4)
    c = P.Context(synth.to_strings(wl["codes"]), wl["theta0"], init_tree=(wl["true_parent"], wl["true_age"]),
                  model=model, kappa=kappa, burnin_steps=1, max_proposals=4, max_samples=8)
    c.mpcgs_sample(4, 8, 11)
    print("n=256", model, c.mpcgs_get_samples()["logL"][:2])
# checkpoint / resume
wl = synth.workload("c2", L=300)
rows = synth.to_strings(wl["codes"])
a = P.Context(rows, wl["theta0"], burnin_steps=2, max_proposals=16, max_samples=64)
a.mpcgs_sample_steps(16, 64, 3, 0, 4)
blob, smp = a.mpcgs_save_state(), a.mpcgs_get_samples()
b = P.Context(rows, wl["theta0"], burnin_steps=2, max_proposals=16, max_samples=64)
b.mpcgs_load_state(blob)
b.mpcgs_put_samples(smp["S"], smp["logL"], smp["step"], smp["slot"])
b.mpcgs_sample_steps(16, 64, 3, 4)
print("resumed", b.mpcgs_num_samples())
print("sanitize run done")
