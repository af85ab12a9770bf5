"""Pick the heaviest top-down and bottom-up level of the first traced root (tools/trace_bfs.py stderr).
Usage: pick_levels.py trace.txt -> prints "TD_LEVEL BU_LEVEL" (level indices = launch indices in the host-driven loop)"""
import re
import sys

td, bu, seen = (0.0, 0), (0.0, 0), 0
for line in open(sys.argv[1]):
    if line.startswith("# root"):
        seen += 1
        if seen > 1:
            break
    m = re.match(r"level\s+(\d+).*\| exp ([\d.]+) bu ([\d.]+)", line)
    if m:
        lv, e, b = int(m.group(1)), float(m.group(2)), float(m.group(3))
        td = max(td, (e, lv))
        bu = max(bu, (b, lv))
print(td[1], bu[1])
