"""Side-by-side per-level spans (us) of GCGT_TRACE logs (first root of each).  Usage: cmp_trace.py a.log b.log ..."""
import re
import sys


def load(path):
    rows = []
    for ln in open(path):
        if ln.startswith("# root") and rows:
            break
        m = re.match(r"level\s+(\d+) next_dir (\d) visited\s+(\d+) new\s+(\d+) next_words\s+(\d+) \| exp ([\d.]+) "
                     r"hub ([\d.]+) bu ([\d.]+) commit ([\d.]+)", ln)
        if m:
            rows.append([float(x) for x in m.groups()])
    return rows


runs = [load(p) for p in sys.argv[1:]]
print("lvl      new  " + " | ".join(f"{'exp':>6} {'hub':>6} {'bu':>6} {'cmt':>6}" for _ in runs))
for i in range(max(len(r) for r in runs)):
    base = runs[0][i] if i < len(runs[0]) else None
    cells = []
    for r in runs:
        cells.append(" ".join(f"{x * 1000:6.1f}" for x in r[i][5:9]) if i < len(r) else " " * 27)
    print(f"{i:3d} {int(base[3]) if base else 0:8d}  " + " | ".join(cells))
tot = [[sum(row[k] for row in r) * 1000 for k in range(5, 9)] for r in runs]
print("sum           " + " | ".join(" ".join(f"{x:6.0f}" for x in t) for t in tot))
