#!/bin/bash
OUT=gpurun_out; mkdir -p $OUT
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py tests/test_gpu_chain.py -m gpu -q -x --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_ch.txt 2>&1; tail -2 $OUT/gpu_tests_ch.txt
bash scripts/gpurun_ab2.sh "ch0" ch 2 "--workload c5
--workload c5 --precision 32
--workload c5 --L 3000
--workload c4 --n 128
--workload c4 --n 256
--workload c3"
