"""Print one compact line of a bench.py JSON output (A/B scripts)."""
import json
import sys

tag, wl, path = sys.argv[1:4]
try:
    d = json.loads(open(path).read().strip().splitlines()[-1])
    print(f"{tag:8s} {wl:28s} {d['value']:.4g} partials/s  {d['ms_per_step']:.4f} ms/step  "
          f"prune {d['roofline']['prune_share_of_step']:.3f}")
except Exception as e:  # noqa: BLE001
    print(f"{tag:8s} {wl:28s} FAILED ({e})")
