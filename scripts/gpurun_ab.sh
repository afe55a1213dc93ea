#!/bin/bash
# interleaved A/B: variants under variants/, c5 FP64, R rounds (bench args via BENCH_ARGS)
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}; R=${2:-2}; shift 2
: > $OUT/ab_$TAG.jsonl
for r in $(seq 1 $R); do
  for v in "$@"; do
    l=$(MPCGS_LIB=variants/libmpcgs_$v.so timeout 300 python bench.py --cpu-seconds 0 --no-e2e --no-incremental-block --steps 10 --warmup 3 ${BENCH_ARGS} 2>/dev/null | tail -1)
    echo "{\"variant\": \"$v\", \"round\": $r, \"line\": $l}" >> $OUT/ab_$TAG.jsonl
  done
done
python - "$OUT/ab_$TAG.jsonl" <<'PY'
import json, sys, collections
d = collections.defaultdict(list)
for l in open(sys.argv[1]):
    x = json.loads(l); d[x["variant"]].append(x["line"]["value"])
for k, v in d.items(): print(k, " ".join("%.4g" % a for a in v))
PY
