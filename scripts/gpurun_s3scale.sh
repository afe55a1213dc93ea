#!/bin/bash
# per-rank scaling emulation at c5 (one GPU: a rank of P scores N/P proposals per step) and A/B of the FP32 F81 cap
OUT=gpurun_out; mkdir -p $OUT; : > $OUT/scale_emul.jsonl
for N in 1024 512 256 128; do
  timeout 300 python bench.py --workload c5 --N $N --cpu-seconds 0 --no-e2e --no-incremental-block --steps 10 2>/dev/null | tail -1 >> $OUT/scale_emul.jsonl
done
python - <<'PY'
import json
rows=[json.loads(l) for l in open("gpurun_out/scale_emul.jsonl")]
t1=rows[0]["ms_per_step"]
for r in rows:
    N=r["config"]["proposals_per_step"]; P=1024//N
    print(f"P={P:2d} N/P={N:5d} ms/step={r['ms_per_step']:.4f} per-rank efficiency={t1/(P*r['ms_per_step']):.3f}")
PY
bash scripts/gpurun_ab2.sh "$1" f32cap 2 "--workload c5 --precision 32
--workload c5 --L 3000 --precision 32
--workload c4 --n 256 --precision 32"
