#!/bin/bash
# GPU tests + compute-sanitizer of the current tree
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}
timeout 1500 python -m pytest tests -m gpu -q --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -3 $OUT/gpu_tests_$TAG.txt
[ "${2:-1}" = 1 ] && bash scripts/gpurun_sanitize.sh $TAG
