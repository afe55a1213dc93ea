#!/bin/bash
# bench sweep over the BASELINE.json configs (1 GPU); one JSON line per point
OUT=gpurun_out/sweep_${1:-x}.jsonl; : > $OUT
run() { timeout 300 python bench.py --cpu-seconds 0 --no-e2e --no-incremental-block --steps ${STEPS:-10} --warmup 3 "$@" 2>/dev/null | tail -1 >> $OUT; }
run --workload c1
run --workload c2
run --workload c3
for n in 8 16 32 64 128 256; do run --workload c4 --n $n; done
for L in 1000 3000 10000 30000 100000; do run --workload c5 --L $L; done
for L in 1000 100000; do run --workload c5 --L $L --precision 32; done
# SURVEY 8(f) variants
run --workload c5 --model F84; run --workload c5 --model F84 --precision 32
run --workload c4 --n 256 --model HKY85 --kappa 4.0
run --workload c5 --ambiguity 0.05; run --workload c5 --ambiguity 0.05 --precision 32
run --workload c5 --incremental; run --workload c5 --compress
wc -l $OUT
