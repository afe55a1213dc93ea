#!/bin/bash
# GPU tests + smoke, the default bench line and the config sweep (no ncu: the captures of
# the unchanged kernels are in profiles/)
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-fin}
timeout 1500 python -m pytest tests -m gpu -q --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -2 $OUT/gpu_tests_$TAG.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke_$TAG.txt 2>&1; tail -1 $OUT/smoke_$TAG.txt
timeout 900 python bench.py > $OUT/bench_c5_$TAG.json 2> $OUT/bench_c5_$TAG.err; tail -1 $OUT/bench_c5_$TAG.json | cut -c1-200
timeout 600 python bench.py --precision 32 --cpu-seconds 0 > $OUT/bench_c5_fp32_$TAG.json 2>/dev/null; tail -1 $OUT/bench_c5_fp32_$TAG.json | cut -c1-200
bash scripts/sweep.sh $TAG
