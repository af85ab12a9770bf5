"""Per-level trace of one profiled BFS (GCGT_TRACE=1 lines on stderr): direction, frontier sizes, span times.
Usage: python tools/trace_bfs.py [config] [nroots]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
os.environ["GCGT_TRACE"] = "1"
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

cfgname = sys.argv[1] if len(sys.argv) > 1 else "c2"
nroots = int(sys.argv[2]) if len(sys.argv) > 2 else 2
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import gcache  # noqa: E402
cfg, ro, cgr, incgr = gcache.graph(cfgname)
g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
roots = synth.pick_roots(ro, 16)
out = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")
g.bfs(roots[0], out=out)  # warm
g.profile(True, spans=True)
for i in range(nroots):
    print(f"# root {roots[i]}", file=sys.stderr, flush=True)
    g.bfs(roots[i], out=out)
    torch.cuda.synchronize()
    print("spans", g.profile_spans(), g.last_stats, file=sys.stderr, flush=True)
