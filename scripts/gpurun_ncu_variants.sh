#!/bin/bash
# ncu --set full of k_prune_tab for each variant under variants/ (WL workload args, FP64 unless PREC set)
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-x}; shift
for v in "$@"; do
  MPCGS_LIB=variants/libmpcgs_$v.so timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_prune_tab -s 3 -c 1 -o $OUT/prof_${TAG}_$v python bench.py $WL --steps 2 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block --precision ${PREC:-64} > $OUT/ncu_${TAG}_$v.log 2>&1; tail -1 $OUT/ncu_${TAG}_$v.log
done
