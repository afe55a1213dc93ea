#!/bin/bash
# fresh-box check: GPU tests + c5 / c2 bench lines
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv
timeout 1200 python -m pytest tests -m gpu -q -x --timeout 600 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -3 $OUT/gpu_tests_$TAG.txt
timeout 600 python bench.py --cpu-seconds 0 > $OUT/bench_c5_$TAG.json 2> $OUT/bench_c5_$TAG.err; tail -1 $OUT/bench_c5_$TAG.json | cut -c1-600
for w in c1 c2 c3; do timeout 300 python bench.py --workload $w --cpu-seconds 0 --no-e2e > $OUT/bench_${w}_$TAG.json 2>/dev/null; tail -1 $OUT/bench_${w}_$TAG.json | cut -c1-300; done
