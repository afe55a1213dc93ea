#!/bin/bash
# validation pass: gpu tests, the default bench line (as the driver runs it), smoke
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv
timeout 1200 python -m pytest tests -m gpu -q --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -3 $OUT/gpu_tests_$TAG.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke_$TAG.txt 2>&1; tail -2 $OUT/smoke_$TAG.txt
timeout 900 python bench.py > $OUT/bench_c5_$TAG.json 2> $OUT/bench_c5_$TAG.err; tail -1 $OUT/bench_c5_$TAG.json | cut -c1-600
