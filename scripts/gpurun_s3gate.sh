#!/bin/bash
OUT=gpurun_out; mkdir -p $OUT
timeout 1500 python -m pytest tests -m gpu -q --timeout 400 -p no:cacheprovider > $OUT/gpu_tests_gate.txt 2>&1; tail -2 $OUT/gpu_tests_gate.txt
bash scripts/gpurun_ab2.sh "ub0" gate 2 "--workload c5
--workload c2
--workload c4 --n 64
--workload c5 --L 1000
--workload c5 --L 30000"
