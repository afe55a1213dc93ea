#!/bin/bash
OUT=gpurun_out/sweep_inc_${1:-x}.jsonl; : > $OUT
run() { timeout 300 python bench.py --cpu-seconds 0 --no-e2e --no-incremental-block --steps ${STEPS:-10} --warmup 3 "$@" 2>/dev/null | tail -1 >> $OUT; }
for inc in "" "--incremental"; do
run --workload c2 $inc
run --workload c3 $inc
for n in 64 256; do run --workload c4 --n $n $inc; done
for L in 1000 100000; do run --workload c5 --L $L $inc; done
done
wc -l $OUT
