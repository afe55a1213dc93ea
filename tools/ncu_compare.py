"""Side-by-side key metrics of several ncu reports (one kernel each)."""
import csv
import subprocess
import sys

KEYS = ["gpu__time_duration.sum", "launch__registers_per_thread", "launch__occupancy_limit_registers",
        "launch__occupancy_limit_shared_mem", "launch__shared_mem_per_block_dynamic", "sm__warps_active.avg.pct_of_peak_sustained_active",
        "smsp__inst_executed.sum", "sm__pipe_fp64_cycles_active.avg.pct_of_peak_sustained_active",
        "smsp__issue_active.avg.pct_of_peak_sustained_active", "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum",
        "l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum", "smsp__sass_inst_executed_op_shared_ld.sum",
        "smsp__sass_inst_executed_op_shared_st.sum", "l1tex__data_pipe_lsu_wavefronts.avg.pct_of_peak_sustained_elapsed",
        "dram__bytes_read.sum"]


def load(rep):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    r = list(csv.reader(out.splitlines()))
    return dict(zip(r[0], r[2]))


reps = [load(r) for r in sys.argv[1:]]
stalls = sorted({k for d in reps for k in d if k.startswith("smsp__average_warps_issue_stalled") and k.endswith("per_issue_active.ratio")})
print(f"{'metric':60s}" + "".join(f"{a.split('/')[-1][:18]:>20s}" for a in sys.argv[1:]))
for k in KEYS + stalls:
    vals = [d.get(k, "") for d in reps]
    try:
        if k in stalls and max(float(v or 0) for v in vals) < 0.1:
            continue
    except ValueError:
        pass
    name = k.replace("smsp__average_warps_issue_stalled_", "stall ").replace("_per_issue_active.ratio", "")
    print(f"{name[:60]:60s}" + "".join(f"{v[:18]:>20s}" for v in vals))
