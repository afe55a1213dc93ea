#!/bin/bash
# sweep each variant (variants/libmpcgs_<v>.so) over the BASELINE configs
for v in "$@"; do MPCGS_LIB=variants/libmpcgs_$v.so STEPS=10 bash scripts/sweep.sh $v > /dev/null; done
for v in "$@"; do echo "== $v"; python tools/sweep_table.py gpurun_out/sweep_$v.jsonl | awk -F'|' 'NR>2{printf "%-40s %s %s\n",$2,$3,$5}'; done
