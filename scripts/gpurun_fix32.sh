mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q 2>&1 | tail -2 > gpurun_out/fix32_tests.txt
bash scripts/gpurun_ab2.sh "lb noslot" fix32 1 "--workload c5 --precision 32
--workload c5
--workload c5 --model F84
--workload c4 --n 128 --precision 32"
