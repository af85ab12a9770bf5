"""§8 f2 — App. D parameter sweeps on B200 (Figs. 11, 12, 14): for each CGR parameter set,
bits per arc (compression) and BFS time / GTEPS on the same synthetic graph.

    python tools/sweep_params.py CONFIG [roots]      -> one JSON line per parameter point
"""
import json
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

name = sys.argv[1]
nroots = int(sys.argv[2]) if len(sys.argv) > 2 else 8
cfg = synth.CONFIGS[name]
ro, co = cfg.make()
m = int(ro[-1])
deg = np.diff(ro.astype(np.int64))
roots = synth.pick_roots(ro, nroots)
points = [("zeta_k (Fig. 11)", (4, 32, k)) for k in (1, 2, 3, 4, 5)]
points += [("min_interval_len (Fig. 12)", (ml, 32, 3)) for ml in (0, 2, 3, 5, 10)]
points += [("residual_segment_len bytes (Fig. 14)", (4, sl, 3)) for sl in (0, 8, 16, 64, 128)]
out = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")
for axis, (ml, sl, k) in points:
    t0 = time.time()
    cgr = G.encode(ro, co, ml, sl, k)
    incgr = None if cfg.symmetric else G.encode_transpose(ro, co, ml, sl, k)
    tenc = time.time() - t0
    _, nbits, _, _, _ = cgr.view()
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
    g.bfs(roots[0], out=out)
    ms, edges = 0.0, 0.0
    for r in roots:
        g.bfs(r, out=out)
        ms += g.last_stats["device_ms"]
        e = float(deg[(out >= 0).cpu().numpy()].sum())
        edges += e / 2 if cfg.symmetric else e
    g.unload()
    print(json.dumps({"config": cfg.name, "axis": axis, "min_interval_len": ml, "residual_segment_len": sl,
                      "zeta_k": k, "bits_per_arc": nbits / m, "compression_vs_32bit": 32 * m / nbits,
                      "bfs_ms": ms / len(roots), "gteps": edges / (ms * 1e-3) / 1e9, "encode_s": round(tenc, 2)}),
          flush=True)
