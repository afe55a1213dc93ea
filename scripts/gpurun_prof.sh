#!/bin/bash
# launch list + ncu --set full of k_prune_tab at c5 (FP64 and FP32), headline step only
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $OUT/launches_c5_$TAG.csv python bench.py --steps 3 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block > /dev/null 2>&1
for p in 64 32; do
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_prune_tab -s 3 -c 1 -o $OUT/prof_prune_c5_fp${p}_$TAG python bench.py --steps 2 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block --precision $p > $OUT/ncu_${TAG}_$p.log 2>&1; tail -1 $OUT/ncu_${TAG}_$p.log
done
