#!/bin/bash
# tests + bench + one ncu capture of k_prune
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}
timeout 900 python -m pytest tests -m gpu -q -x --timeout 300 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -3 $OUT/gpu_tests_$TAG.txt
timeout 600 python bench.py --cpu-seconds 0 --no-e2e > $OUT/bench_c5_$TAG.json 2>&1; tail -1 $OUT/bench_c5_$TAG.json | cut -c1-400
timeout 600 python bench.py --precision 32 --cpu-seconds 0 --no-e2e > $OUT/bench_c5f32_$TAG.json 2>&1; tail -1 $OUT/bench_c5f32_$TAG.json | cut -c1-300
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_prune_tab -s 3 -c 1 -o $OUT/prof_prune_$TAG python bench.py --steps 2 --warmup 3 --no-e2e --cpu-seconds 0 > $OUT/ncu_$TAG.log 2>&1; tail -1 $OUT/ncu_$TAG.log
