#!/bin/bash
OUT=gpurun_out/sweep_${1:-x}.jsonl; : > $OUT
run() { timeout 300 python bench.py --cpu-seconds 0 --no-e2e --no-incremental-block --steps 10 --warmup 3 "$@" 2>/dev/null | tail -1 >> $OUT; }
for th in 1.0 0.01; do for comp in "" "--compress"; do
run --workload c5 --L 100000 --theta-true $th $comp
run --workload c2 --theta-true $th $comp
done; done
