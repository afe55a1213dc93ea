"""Summarise an ncu launch list (--metrics gpu__time_duration.sum --csv): per kernel the
launch count, mean device time, and its share of the GMH-step kernels' time.  The
roofline microbenchmarks bench.py runs before its timed region (k_fma, k_lds of
csrc/probe.cu) and the one-time init kernel (k_unpack_codes) are listed but excluded
from the step shares.  The times are ncu's (cold-cache, serialised): compare shares."""
import csv
import sys
from collections import defaultdict

NOT_STEP = ("k_fma", "k_lds", "k_unpack_codes")
AFTER = ("k_theta_grid", "k_theta_moments", "k_minmax")  # theta MLE (row a7), once after sampling
rows = list(csv.reader(open(sys.argv[1])))
hdr = next(i for i, r in enumerate(rows) if 'Kernel Name' in r)
h = rows[hdr]
ki, vi = h.index('Kernel Name'), h.index('Metric Value')
d = defaultdict(list)
for r in rows[hdr + 1:]:
    if len(r) > vi:
        d[r[ki][:60]].append(float(r[vi].replace(',', '')))
step = {k: v for k, v in d.items() if not any(x in k for x in NOT_STEP + AFTER)}
tot = sum(sum(v) for v in step.values())
for k, v in sorted(d.items(), key=lambda kv: -sum(kv[1])):
    share = (f"step share={sum(v) / tot:6.3f}" if k in step else
             "(theta MLE after sampling, M = 1e6)" if any(x in k for x in AFTER) else "(not a step kernel)")
    med = sorted(v)[len(v) // 2]
    print(f"{k:60s} n={len(v):4d} mean={sum(v) / len(v) / 1e3:9.2f} us  median={med / 1e3:9.2f} us  {share}")
