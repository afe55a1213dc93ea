#!/bin/bash
# session-3 A/B: product tables at n = 256 FP64 (pt256), 2 sites per thread from n = 97 (ws96)
OUT=gpurun_out; mkdir -p $OUT
bash scripts/gpurun_ab2.sh "$1" ${2:-ws} ${3:-2} "--workload c4 --n 256
--workload c4 --n 192
--workload c4 --n 128
--workload c4 --n 128 --precision 32
--workload c4 --n 256 --model HKY85 --kappa 4.0
--workload c5 --L 10000 --n 128"
