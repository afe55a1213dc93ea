#!/bin/bash
# session-3 A/B of the table-kernel smem layout (aliasing, single code buffer)
OUT=gpurun_out; mkdir -p $OUT; TAG=${2:-lay}; R=${3:-2}; T=${4:-1}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv,noheader
if [ "$T" = 1 ]; then
timeout 1500 python -m pytest tests -m gpu -q -x --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -3 $OUT/gpu_tests_$TAG.txt
fi
bash scripts/gpurun_ab2.sh "$1" $TAG $R "--workload c5
--workload c4 --n 256
--workload c4 --n 192
--workload c4 --n 128
--workload c4 --n 256 --precision 32
--workload c4 --n 256 --model HKY85 --kappa 4.0
--workload c5 --precision 32
--workload c5 --L 3000"
