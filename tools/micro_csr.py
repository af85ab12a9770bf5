"""CGR vs uncompressed-CSR BFS (§8 f3) on one config: device ms per BFS over the same roots, both top-down only and
direction-optimizing.  Usage: python tools/micro_csr.py CONFIG NROOTS"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

cfgname, nroots = sys.argv[1], int(sys.argv[2])
cfg = synth.CONFIGS[cfgname]
ro, co = cfg.make()
P = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
cgr = G.encode(ro, co, *P)
incgr = None if cfg.symmetric else G.encode_transpose(ro, co, *P)
roots = synth.pick_roots(ro, nroots)
out = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")


def run(g):
    g.bfs(roots[0], out=out)
    ms, edges = [], 0
    ref = []
    for r in roots:
        g.bfs(r, out=out)
        ms.append(g.last_stats["device_ms"])
        ref.append(int(out.sum().item()))
    return sum(ms) / len(ms), ref


for dopt in (False, True):
    gc = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric, direction_optimizing=dopt)
    tc, rc = run(gc)
    gc.unload()
    gs = G.load_csr(ro, co, stream="torch", symmetric=cfg.symmetric, direction_optimizing=dopt)
    ts, rs = run(gs)
    gs.unload()
    print(f"{cfgname} dir_opt={int(dopt)}  CGR {tc:8.3f} ms  CSR {ts:8.3f} ms  CGR/CSR {tc / ts:5.2f}  "
          f"{'ok' if rc == rs else 'MISMATCH'}", flush=True)
