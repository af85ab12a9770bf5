"""CC and BC timings on the BASELINE configs (companion to bench.py, which times BFS, the headline metric).

    python tools/bench_apps.py cc c2 [reps]          # weakly connected components on the uk-2002-like graph
    python tools/bench_apps.py bc c3 [nsrc]          # betweenness centrality, 64 seeded sources, twitter-like graph
    python tools/bench_apps.py bfs c3 [reps]         # BFS on another config

Prints one JSON line: device ms per call (CUDA events inside the library), arcs decoded, and a sampled parity check
against the oracle (full CC labels; BC from 1 source; BFS from 1 root).
"""
import json
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import oracle as O  # noqa: E402
import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

app, name = sys.argv[1], sys.argv[2]
arg = int(sys.argv[3]) if len(sys.argv) > 3 else None
cfg = synth.CONFIGS[name]
t0 = time.time()
ro, co = cfg.make()
tgen = time.time() - t0
P = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
t0 = time.time()
cgr = G.encode(ro, co, *P)
tenc = time.time() - t0
_, nbits, _, n, _ = cgr.view()
m = int(ro[-1])
out = {"app": app, "config": cfg.name + ": " + cfg.desc, "n": int(n), "m": m, "bits_per_arc": nbits / max(m, 1),
       "gen_s": round(tgen, 1), "encode_s": round(tenc, 1)}
if app == "cc":
    g = G.load(cgr, stream="torch")
    reps = arg or 5
    dlab = torch.empty(int(n), dtype=torch.int32, device="cuda")  # device output: device_ms excludes the D2H
    g.cc(out=dlab)
    ms = []
    for _ in range(reps):
        g.cc(out=dlab)
        ms.append(g.last_stats["device_ms"])
    lab = dlab.cpu().numpy().view(np.uint32)
    out.update({"ms": float(np.median(ms)), "reps": reps, "stats": g.last_stats,
                "arcs_per_s_G": m / (np.median(ms) * 1e-3) / 1e9})
    t0 = time.time()
    ref = O.cc(ro, co)
    out["oracle_s"] = round(time.time() - t0, 2)
    out["parity"] = bool(np.array_equal(lab, ref))
    out["components"] = int(np.unique(ref).size)
elif app == "bc":
    incgr = None
    g = G.load(cgr, stream="torch")
    nsrc = arg or 64
    src = synth.bc_sources(ro, nsrc)
    g.bc(src[:2])  # warm-up
    bc = g.bc(src)
    st = g.last_stats
    out.update({"sources": nsrc, "ms": st["device_ms"], "ms_per_source": st["device_ms"] / nsrc, "stats": st})
    # sampled parity: the first source alone against the oracle's Brandes
    one = g.bc(src[:1])
    t0 = time.time()
    ref = O.bc(ro, co, src[:1])
    out["oracle_s_per_source"] = round(time.time() - t0, 2)
    ok = np.array_equal(one == 0, ref == 0) and np.allclose(one, ref, rtol=1e-9, atol=0)
    out["parity_1_source"] = bool(ok)
    out["max_rel_err_1_source"] = float(np.max(np.abs(one - ref) / np.maximum(np.abs(ref), 1e-300)))
else:
    incgr = None if cfg.symmetric else G.encode_transpose(ro, co, *P)
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
    roots = synth.pick_roots(ro, arg or 8)
    deg = np.diff(ro.astype(np.int64))
    ms, edges = [], 0
    dlv = torch.empty(int(n), dtype=torch.int32, device="cuda")  # device output: device_ms excludes the D2H
    g.bfs(roots[0], out=dlv)
    for r in roots:
        g.bfs(r, out=dlv)
        ms.append(g.last_stats["device_ms"])
        lv = dlv.cpu().numpy()
        e = int(deg[lv >= 0].sum())
        edges += e / 2 if cfg.symmetric else e
    out.update({"roots": len(roots), "ms_per_bfs": float(np.mean(ms)), "ms_each": [round(x, 3) for x in ms],
                "gteps": edges / (sum(ms) * 1e-3) / 1e9, "levels_on": "device"})
    out["parity_1_root"] = bool(np.array_equal(lv, O.bfs(ro, co, roots[-1])))
print(json.dumps(out), flush=True)
