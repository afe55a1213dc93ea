#!/bin/bash
# ncu --set full of the small-config step kernels (c2): k_propose, k_draw, k_context
OUT=gpurun_out; mkdir -p $OUT
for k in k_propose k_draw k_prune_tab; do
timeout 600 ncu --set full --clock-control none --import-source on -k regex:$k -s 5 -c 1 -o $OUT/prof_c2_$k python bench.py --workload c2 --steps 4 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block > $OUT/ncu_c2_$k.log 2>&1; tail -1 $OUT/ncu_c2_$k.log
done
