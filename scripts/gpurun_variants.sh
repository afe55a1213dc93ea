#!/bin/bash
# A/B the tuning variants under variants/ on c5 (FP64 + FP32); then the GPU tests on the default build
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}; shift
: > $OUT/var_$TAG.jsonl
for v in "$@"; do
  for p in 64 32; do
    r=$(MPCGS_LIB=variants/libmpcgs_$v.so timeout 300 python bench.py --cpu-seconds 0 --no-e2e --no-incremental-block --steps 10 --warmup 3 --precision $p 2>/dev/null | tail -1)
    echo "{\"variant\": \"$v\", \"precision\": $p, \"line\": $r}" >> $OUT/var_$TAG.jsonl
    echo "$v fp$p $(echo $r | cut -c90-160)"
  done
done
timeout 900 python -m pytest tests -m gpu -q -x --timeout 300 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -3 $OUT/gpu_tests_$TAG.txt
