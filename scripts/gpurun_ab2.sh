#!/bin/bash
# interleaved A/B of bench lines: in-tree library ("new") vs variants/libmpcgs_<v>.so
# usage: gpurun_ab2.sh "v1 v2" TAG ROUNDS "workload lines (\n separated)"
OUT=gpurun_out; mkdir -p $OUT; TAG=${2:-x}; R=${3:-2}
WL=${4:-"--workload c5
--workload c5 --L 3000
--workload c3
--workload c2
--workload c4 --n 256"}
LOG=$OUT/ab_$TAG.log; : > $LOG
for r in $(seq $R); do
while read -r w; do
  for v in new $1; do
    if [ $v = new ]; then export MPCGS_LIB=; unset MPCGS_LIB; else export MPCGS_LIB=variants/libmpcgs_$v.so; fi
    timeout 300 python bench.py $w --cpu-seconds 0 --no-e2e --no-incremental-block --steps 10 > $OUT/ab_line.json 2>> $LOG
    python tools/ab_line.py "$v" "$w" $OUT/ab_line.json | tee -a $OUT/ab_$TAG.txt
  done
done <<< "$WL"
done
unset MPCGS_LIB
