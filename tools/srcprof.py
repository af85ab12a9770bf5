"""Aggregates an ncu source page (--print-source cuda,sass --csv) per CUDA source line:
warp-level instructions executed, thread instructions, stall samples.  Usage: srcprof.py report.ncu-rep [top]"""
import csv
import subprocess
import sys

rep = sys.argv[1]
top = int(sys.argv[2]) if len(sys.argv) > 2 else 40
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "cuda,sass"],
                     capture_output=True, text=True).stdout.splitlines()
agg = {}
srcs = {}
cur_file = ""
tot_i = tot_s = 0
hdr = None
for row in csv.reader(out):
    if not row:
        continue
    if row[0] == "File Path":
        cur_file = row[1].split("/")[-1]
        continue
    if row[0] == "Line No":
        hdr = row
        continue
    if hdr is None or row[0] in ("Function Name",):
        continue
    try:
        line = int(row[0])
    except ValueError:
        continue
    d = dict(zip(hdr[2:], row[2:]))
    try:
        wi = int(d.get("Instructions Executed", "0") or 0)
        ti = int(d.get("Thread Instructions Executed", "0") or 0)
        sm = int(d.get("Warp Stall Sampling (All Samples)", "0") or 0)
    except ValueError:
        continue
    key = (cur_file, line)
    a = agg.setdefault(key, [0, 0, 0])
    a[0] += wi
    a[1] += ti
    a[2] += sm
    srcs[key] = row[1][:70]
    tot_i += wi
    tot_s += sm
print(f"total warp instr {tot_i}, stall samples {tot_s}")
for key, (wi, ti, sm) in sorted(agg.items(), key=lambda x: -x[1][0])[:top]:
    print(f"{key[0]:12s}:{key[1]:<5d} instr {wi:10d} ({wi / tot_i:5.1%}) thr/instr {ti / max(wi, 1):5.1f} "
          f"stall {sm / max(tot_s, 1):5.1%}  {srcs[key].strip()}")
