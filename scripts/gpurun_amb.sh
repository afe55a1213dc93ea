mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_bench.py -x -q 2>&1 | tail -5 > gpurun_out/amb_tests.txt
bash scripts/gpurun_ab2.sh "base" amb 1 "--workload c5 --ambiguity 0.05
--workload c4 --n 256 --ambiguity 0.05
--workload c2 --ambiguity 0.05
--workload c5 --ambiguity 0.05 --precision 32"
