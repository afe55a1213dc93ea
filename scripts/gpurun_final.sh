#!/bin/bash
# GPU tests + smoke, then the evidence set (bench line, FP32 line, launch list, ncu captures, sweep)
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-fin}
timeout 1500 python -m pytest tests -m gpu -q --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_$TAG.txt 2>&1; tail -2 $OUT/gpu_tests_$TAG.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke_$TAG.txt 2>&1; tail -1 $OUT/smoke_$TAG.txt
bash scripts/gpurun_evidence3.sh $TAG 1
