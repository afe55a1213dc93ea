mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py tests/test_gpu_chain.py -x -q 2>&1 | tail -3 > gpurun_out/slot3_tests.txt
bash scripts/gpurun_ab2.sh "noslot" slot3 1 "--workload c5
--workload c5 --model F84
--workload c5 --model F84 --precision 32
--workload c4 --n 128 --model HKY85
--workload c5 --model F84 --ambiguity 0.05"
