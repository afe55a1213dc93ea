#!/bin/bash
# round-2 evidence: bench line (default command), launch list, ncu --set full of the dominant
# kernels, config sweep
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}; SWEEP=${2:-1}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv
timeout 900 python bench.py > $OUT/bench_c5_$TAG.json 2> $OUT/bench_c5_$TAG.err; tail -1 $OUT/bench_c5_$TAG.json | cut -c1-200
timeout 600 python bench.py --precision 32 --cpu-seconds 0 > $OUT/bench_c5_fp32_$TAG.json 2>/dev/null; tail -1 $OUT/bench_c5_fp32_$TAG.json | cut -c1-200
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $OUT/launches_c5_$TAG.csv python bench.py --steps 3 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block > /dev/null 2>&1
for p in 64 32; do
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_prune_tab -s 3 -c 1 -o $OUT/prof_prune_c5_fp${p}_$TAG python bench.py --steps 2 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block --precision $p > $OUT/ncu_${TAG}_$p.log 2>&1; tail -1 $OUT/ncu_${TAG}_$p.log
done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_score_incr -s 3 -c 1 -o $OUT/prof_incr_c5_fp64_$TAG python bench.py --steps 2 --warmup 3 --no-e2e --cpu-seconds 0 --incremental > $OUT/ncu_${TAG}_incr.log 2>&1; tail -1 $OUT/ncu_${TAG}_incr.log
[ "$SWEEP" = 1 ] && bash scripts/sweep.sh $TAG
