"""Summarise an ncu --csv launch list (gpu__time_duration.sum [+ dram__bytes_read/write.sum]): per kernel
launch count, total time, share, DRAM bytes.  Usage: launches.py list.csv [--seq] [--json out.json]"""
import collections
import csv
import json
import sys


def load(path):
    with open(path) as f:
        lines = [ln for ln in f if not ln.startswith("==")]
    return list(csv.DictReader(lines))


def main(path, show_seq=False, json_out=None):
    rows = load(path)
    per = collections.OrderedDict()
    for r in rows:
        key = (r["ID"], r["Kernel Name"].replace("<unnamed>::", "").replace("(anonymous namespace)::", ""))
        d = per.setdefault(key, {"grid": r.get("Grid Size", "")})
        unit = r["Metric Unit"]
        val = float(r["Metric Value"].replace(",", ""))
        if r["Metric Name"] == "gpu__time_duration.sum":
            d["us"] = val / 1e3 if unit == "nsecond" or unit == "ns" else val
        elif r["Metric Name"].startswith("dram__bytes"):
            scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}.get(unit, 1)
            d["dram"] = d.get("dram", 0.0) + val * scale
    agg = collections.defaultdict(lambda: [0, 0.0, 0.0])
    for (i, name), d in per.items():
        short = name.split("(")[0]
        agg[short][0] += 1
        agg[short][1] += d.get("us", 0.0)
        agg[short][2] += d.get("dram", 0.0)
    tot = sum(v[1] for v in agg.values())
    print(f"{'kernel':66s} {'n':>4s} {'total_us':>10s} {'share':>6s} {'dram_MB':>9s}")
    for k, v in sorted(agg.items(), key=lambda x: -x[1][1]):
        print(f"{k[:66]:66s} {v[0]:4d} {v[1]:10.1f} {v[1] / tot:6.3f} {v[2] / 1e6:9.1f}")
    print(f"total {tot:.1f} us over {len(per)} launches")
    if show_seq:
        for (i, name), d in per.items():
            print(i, name.split("(")[0][:60], d)
    if json_out:
        with open(json_out, "w") as f:
            json.dump({k: {"launches": v[0], "us": v[1], "dram_bytes": v[2]} for k, v in agg.items()}, f, indent=1)


if __name__ == "__main__":
    jo = sys.argv[sys.argv.index("--json") + 1] if "--json" in sys.argv else None
    main(sys.argv[1], "--seq" in sys.argv, jo)
