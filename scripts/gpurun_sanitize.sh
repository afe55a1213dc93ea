#!/bin/bash
# compute-sanitizer memcheck / racecheck / synccheck over every kernel (tools/sanitize_run.py)
OUT=gpurun_out; mkdir -p $OUT; F=$OUT/sanitizer_${1:-x}.txt
echo "# compute-sanitizer on tools/sanitize_run.py (all kernels, FP64/FP32, full/incremental, c1 and n=128)" > $F
for t in memcheck racecheck synccheck; do
  echo "## $t" >> $F
  timeout 1200 compute-sanitizer --tool $t python tools/sanitize_run.py >> $F 2>&1
done
grep -E "SUMMARY|sanitize run done" $F
