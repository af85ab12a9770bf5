"""Times gcgt_load / gcgt_bfs (host output) / gcgt_unload separately on a config (diagnostics for bench e2e)."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

cfg = synth.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "c2"]
ro, co = cfg.make()
P = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
cgr = G.encode(ro, co, *P)
incgr = None if cfg.symmetric else G.encode_transpose(ro, co, *P)  # as bench.py e2e
iters = int(sys.argv[2]) if len(sys.argv) > 2 else 3
root = synth.pick_roots(ro, 1)[0]
levels = torch.empty(ro.size - 1, dtype=torch.int32).pin_memory()
for i in range(iters):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
    torch.cuda.synchronize()
    t1 = time.perf_counter()
    g.bfs(root, out=levels)
    t2 = time.perf_counter()
    g.unload()
    torch.cuda.synchronize()
    t3 = time.perf_counter()
    print(f"load {1e3*(t1-t0):.1f} ms  bfs {1e3*(t2-t1):.1f} ms  unload {1e3*(t3-t2):.1f} ms  stats {g.last_stats}")
