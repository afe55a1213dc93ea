#!/bin/bash
# session-3 A/B: GPU tests of the in-tree library, then interleaved bench A/B vs variants
# usage: gpurun_s3ab.sh "variants" TAG ROUNDS [tests: 1/0]
OUT=gpurun_out; mkdir -p $OUT; TAG=${2:-x}; R=${3:-2}; T=${4:-1}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv,noheader
if [ "$T" = 1 ]; then
timeout 1500 python -m pytest tests -m gpu -q -x --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -3 $OUT/gpu_tests_$TAG.txt
fi
bash scripts/gpurun_ab2.sh "$1" $TAG $R "--workload c5
--workload c5 --L 3000
--workload c3
--workload c4 --n 128
--workload c4 --n 256
--workload c5 --precision 32"
