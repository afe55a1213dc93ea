"""Aggregate ncu warp-stall samples of one kernel by CUDA source line.
usage: python tools_linesamples.py REPORT.ncu-rep CUBIN MANGLED_NAME [top]"""
import csv, os, re, subprocess, sys
from collections import defaultdict
rep, cubin, fn = sys.argv[1:4]
top = int(sys.argv[4]) if len(sys.argv) > 4 else 30
dis = subprocess.run(["nvdisasm", "-g", "-c", cubin], capture_output=True, text=True).stdout
sec = dis.split(f".text.{fn}:")[1].split("//---------------------")[0]
off2line, cur = {}, None
for ln in sec.splitlines():
    m = re.search(r'File "([^"]+)", line (\d+)', ln)
    if m:
        cur = (m.group(1).split("/")[-1], int(m.group(2)))
        continue
    m = re.match(r"\s+/\*([0-9a-f]{4,})\*/", ln)
    if m and cur:
        off2line[int(m.group(1), 16)] = cur
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv"], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]; data = rows[2:]
ai, si, ie = h.index("Address"), h.index("Warp Stall Sampling (All Samples)"), h.index("Instructions Executed")
base = min(int(r[ai], 16) for r in data)
agg, inst = defaultdict(float), defaultdict(float)
for r in data:
    key = off2line.get(int(r[ai], 16) - base, ("?", 0))
    agg[key] += float(r[si] or 0)
    inst[key] += float(r[ie] or 0)
tot = sum(agg.values())
src = {}
for (f, l) in agg:
    try:
        src[(f, l)] = open(os.environ.get("SRCDIR", "paper_conf_ipps_davistzw17_b200/csrc") + f"/{f}").read().splitlines()[l - 1].strip()[:70]
    except Exception:
        src[(f, l)] = ""
for k, v in sorted(agg.items(), key=lambda kv: -kv[1])[:top]:
    print(f"{v/tot:6.3f} {int(inst[k]):9d} {k[0]}:{k[1]:<5d} {src[k]}")
