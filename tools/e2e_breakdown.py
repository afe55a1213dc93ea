"""Wall-clock breakdown of bench.py's end-to-end leg (public API from host buffers)."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_ipps_davistzw17_b200 as P  # noqa: E402

wl = synth.workload("c5")
rows = synth.to_strings(wl["codes"])
N, steps = wl["N"], 20
stream = torch.cuda.current_stream().cuda_stream
for rep in range(3):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    c = P.Context(rows, wl["theta0"], max_proposals=N, max_samples=N * steps,
                  init_tree=(wl["true_parent"], wl["true_age"]), stream=stream)
    t1 = time.perf_counter()
    c.mpcgs_sample(N, N * steps, wl["chain_seed"] + 1)
    t2 = time.perf_counter()
    smp = c.mpcgs_get_samples()
    t3 = time.perf_counter()
    c.free()
    t4 = time.perf_counter()
    print(f"rep {rep}: init {1e3*(t1-t0):.1f} ms, sample({steps} steps) {1e3*(t2-t1):.1f} ms, "
          f"get_samples {1e3*(t3-t2):.1f} ms, free {1e3*(t4-t3):.1f} ms", flush=True)
