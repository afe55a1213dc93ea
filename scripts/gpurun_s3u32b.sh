#!/bin/bash
OUT=gpurun_out; mkdir -p $OUT
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py tests/test_gpu_multirank.py -m gpu -q --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_u32b.txt 2>&1; tail -2 $OUT/gpu_tests_u32b.txt
bash scripts/gpurun_ab2.sh "u32off" u32b 2 "--workload c5 --precision 32
--workload c5 --L 30000 --precision 32
--workload c5"
