mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q 2>&1 | tail -3 > gpurun_out/lb_tests.txt
bash scripts/gpurun_ab2.sh "base" lb 1 "--workload c5 --model F84
--workload c5
--workload c5 --precision 32
--workload c4 --n 256 --model HKY85
--workload c4 --n 256
--workload c3"
