#!/bin/bash
# final evidence: bench lines, launch list, ncu --set full of the FP64 prune kernel, sweep, smoke
OUT=gpurun_out; mkdir -p $OUT; TAG=${1:-fin}
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke_$TAG.txt 2>&1; tail -1 $OUT/smoke_$TAG.txt
timeout 900 python bench.py > $OUT/bench_c5_$TAG.json 2> $OUT/bench_c5_$TAG.err; tail -1 $OUT/bench_c5_$TAG.json | cut -c1-200
timeout 600 python bench.py --precision 32 --cpu-seconds 0 > $OUT/bench_c5_fp32_$TAG.json 2>/dev/null; tail -1 $OUT/bench_c5_fp32_$TAG.json | cut -c1-200
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $OUT/launches_c5_$TAG.csv python bench.py --steps 3 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_prune_tab -s 3 -c 1 -o $OUT/prof_prune_c5_fp64_$TAG python bench.py --steps 2 --warmup 3 --no-e2e --cpu-seconds 0 --no-incremental-block > $OUT/ncu_${TAG}_64.log 2>&1; tail -1 $OUT/ncu_${TAG}_64.log
bash scripts/sweep.sh $TAG
