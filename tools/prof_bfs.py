"""One-shot driver for ncu: builds config graph, loads it, runs `reps` BFS (and optionally CC / BC) on cuda:0."""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--config", default="c2")
ap.add_argument("--reps", type=int, default=1)
ap.add_argument("--app", default="bfs", choices=["bfs", "cc", "bc"])
ap.add_argument("--bc-sources", type=int, default=1)
a = ap.parse_args()
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import gcache  # noqa: E402
cfg, ro, cgr, incgr = gcache.graph(a.config)
g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
roots = synth.pick_roots(ro, 16)
out = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")
for i in range(a.reps):
    if a.app == "bfs":
        g.bfs(roots[i % len(roots)], out=out)
    elif a.app == "cc":
        g.cc(out=out)
    else:
        g.bc(synth.bc_sources(ro, a.bc_sources))
    print(a.app, g.last_stats, flush=True)
torch.cuda.synchronize()
