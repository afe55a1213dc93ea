mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q 2>&1 | tail -3 > gpurun_out/slot_tests.txt
bash scripts/gpurun_ab2.sh "noslot" slot 2 "--workload c5
--workload c5 --precision 32
--workload c5 --model F84
--workload c5 --L 3000
--workload c3
--workload c4 --n 256"
