#!/bin/bash
# one GPU session: tests, bench, ncu launch list and full capture of the top kernel
set -x
OUT=gpurun_out
mkdir -p $OUT
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv
timeout 900 python -m pytest tests -m gpu -q --timeout 300 -p no:cacheprovider > $OUT/gpu_tests.txt 2>&1; tail -5 $OUT/gpu_tests.txt
timeout 600 python bench.py > $OUT/bench_c5.json 2> $OUT/bench_c5.err; tail -2 $OUT/bench_c5.json; tail -3 $OUT/bench_c5.err
timeout 600 python bench.py --workload c2 --cpu-seconds 5 > $OUT/bench_c2.json 2> $OUT/bench_c2.err; tail -1 $OUT/bench_c2.json
timeout 600 python bench.py --precision 32 --cpu-seconds 0 > $OUT/bench_c5_fp32.json 2>&1; tail -1 $OUT/bench_c5_fp32.json
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $OUT/launches_c5.csv python bench.py --steps 3 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_prune_tab -s 3 -c 1 -o $OUT/prof_prune_c5 python bench.py --steps 2 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block > $OUT/ncu_full.log 2>&1; tail -3 $OUT/ncu_full.log
ls -la $OUT
