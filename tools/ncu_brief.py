"""Key metrics of an ncu --set full report (one kernel), read on the box so the .ncu-rep need not travel back.
Usage: python tools/ncu_brief.py report.ncu-rep > summary.txt"""
import csv
import subprocess
import sys

KEYS = ["Kernel Name", "Grid Size", "Block Size", "gpu__time_duration.sum", "dram__bytes_read.sum",
        "dram__bytes_write.sum", "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed",
        "sm__throughput.avg.pct_of_peak_sustained_elapsed", "sm__warps_active.avg.pct_of_peak_sustained_active",
        "smsp__thread_inst_executed_per_inst_executed.ratio", "launch__registers_per_thread",
        "launch__occupancy_limit_registers", "sm__maximum_warps_per_active_cycle_pct",
        "l1tex__t_sector_hit_rate.pct", "lts__t_sector_hit_rate.pct", "smsp__issue_active.avg.pct_of_peak_sustained_active",
        "sm__cycles_active.avg", "gpc__cycles_elapsed.max", "smsp__inst_executed.sum",
        "smsp__average_warp_latency_issue_stalled_long_scoreboard", "smsp__average_warp_latency_issue_stalled_short_scoreboard",
        "smsp__average_warp_latency_issue_stalled_wait", "smsp__average_warp_latency_issue_stalled_barrier",
        "smsp__average_warp_latency_issue_stalled_lg_throttle", "smsp__average_warp_latency_issue_stalled_no_instruction",
        "smsp__average_warp_latency_issue_stalled_math_pipe_throttle", "smsp__average_warp_latency_issue_stalled_membar",
        "smsp__average_warp_latency_issue_stalled_branch_resolving", "smsp__average_warp_latency_issue_stalled_dispatch_stall",
        "smsp__average_warp_latency_issue_stalled_not_selected", "smsp__average_warp_latency_issue_stalled_selected",
        "smsp__average_warp_latency_issue_stalled_mio_throttle", "smsp__average_warp_latency_issue_stalled_drain",
        "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum", "lts__t_requests_srcunit_tex_op_atom.sum",
        "lts__t_requests_srcunit_tex_op_red.sum"]

rep = sys.argv[1]
out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout.splitlines()
rows = list(csv.reader(out))
if len(rows) < 3:
    print("no data", out[:5])
    sys.exit(0)
hdr, units = rows[0], rows[1]
for r in rows[2:]:
    for k in KEYS:
        for i, h in enumerate(hdr):
            if h == k or (k.startswith("smsp__average_warp_latency") and h.startswith(k)):
                print(f"{h[:72]:72s} {units[i][:10]:10s} {r[i][:60]}")
                break
    print()
