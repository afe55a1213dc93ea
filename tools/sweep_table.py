"""Markdown table of bench.py JSON lines (one per line) for profiles/."""
import json
import sys

print("| workload | dtype | model | scoring | partials/s | proposals/s | ms/step | prune share | prune frac |")
print("|---|---|---|---|---|---|---|---|---|")
for path in sys.argv[1:]:
    for line in open(path):
        d = json.loads(line)
        c, r = d["config"], d.get("roofline") or {}
        frac = r.get("frac")
        model = c.get("model", "F81") + (" + IUPAC" if c.get("ambiguity", "none") != "none" else "")
        print(f"| {c['workload'].split(',')[0]} | {d['dtype']} | {model} | {c.get('scoring', '').split(' (')[0]} | {d['value']:.3g} | "
              f"{d['proposals_per_s']:.3g} | {d['ms_per_step']:.3f} | {r.get('prune_share_of_step', 0):.2f} | "
              f"{'-' if frac is None else f'{frac:.3f}'} |")
