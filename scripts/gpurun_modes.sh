#!/bin/bash
# every bench.py mode once (c5 unless noted), one JSON line each
OUT=gpurun_out/modes_${1:-x}.jsonl; : > $OUT
run() { timeout 300 python bench.py --cpu-seconds 0 --no-e2e --steps 5 --warmup 3 "$@" 2>&1 | tail -1 >> $OUT; }
run --model F84
run --model HKY85 --workload c4 --n 256
run --model F84 --precision 32
run --compress --theta-true 0.01
run --incremental
run --ambiguity 0.01
run --loci 4 --workload c3
run --workload c4 --n 256
run --workload c1
python - $OUT <<'PY'
import json, sys
for l in open(sys.argv[1]):
    try:
        d = json.loads(l); c = d.get("config", {})
        print(c.get("workload", "?")[:40], c.get("model"), c.get("scoring", "")[:20], d.get("dtype"), "%.3g" % d["value"], (d.get("roofline") or {}).get("frac"))
    except Exception as e:
        print("BAD:", l[:200])
PY
