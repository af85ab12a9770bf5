"""Summarise an ncu --metrics gpu__time_duration.sum --csv launch list: per-kernel count / time / share."""
import collections
import csv
import sys


def load(path):
    with open(path) as f:
        lines = [ln for ln in f if not ln.startswith("==")]
    return list(csv.DictReader(lines))


def main(path, show_seq=False):
    rows = load(path)
    agg = collections.defaultdict(lambda: [0, 0.0])
    seq = []
    for r in rows:
        name = r["Kernel Name"].replace("<unnamed>::", "").replace("(anonymous namespace)::", "")
        short = name.split("(")[0]
        t = float(r["Metric Value"]) / 1e3
        agg[short][0] += 1
        agg[short][1] += t
        seq.append((short[:60], t, r["Grid Size"]))
    tot = sum(v[1] for v in agg.values())
    print(f"{'kernel':70s} {'n':>4s} {'total_us':>10s} {'share':>6s}")
    for k, v in sorted(agg.items(), key=lambda x: -x[1][1]):
        print(f"{k[:70]:70s} {v[0]:4d} {v[1]:10.1f} {v[1] / tot:6.3f}")
    print(f"total {tot:.1f} us over {len(rows)} launches")
    if show_seq:
        for s in seq:
            print(s)


if __name__ == "__main__":
    main(sys.argv[1], "--seq" in sys.argv)
