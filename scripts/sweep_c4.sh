#!/bin/bash
OUT=gpurun_out/sweep_${1:-x}.jsonl; : > $OUT
run() { timeout 300 python bench.py --cpu-seconds 0 --no-e2e --no-incremental-block --steps ${STEPS:-10} --warmup 3 "$@" 2>/dev/null | tail -1 >> $OUT; }
for n in 64 128 256; do run --workload c4 --n $n; done
run --workload c5
