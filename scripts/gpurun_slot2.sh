mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q 2>&1 | tail -3 > gpurun_out/slot2_tests.txt
bash scripts/gpurun_ab2.sh "noslot" slot2 1 "--workload c5
--workload c5 --model F84
--workload c5 --model F84 --precision 32
--workload c4 --n 128 --model HKY85
--workload c4 --n 256 --model HKY85
--workload c5 --model F84 --ambiguity 0.05
--workload c3 --model F84"
