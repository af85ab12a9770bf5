"""Times BFS on a config for several GCGT_TUNE settings (one process; the knobs are read at gcgt_load)."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

cfg = synth.CONFIGS[sys.argv[1]]
tunes = sys.argv[2:]
ro, co = cfg.make()
P = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
cgr = G.encode(ro, co, *P)
incgr = None if cfg.symmetric else G.encode_transpose(ro, co, *P)
roots = synth.pick_roots(ro, 8)
out = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")
for tune in tunes:
    os.environ["GCGT_TUNE"] = tune
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
    for r in roots[:2]:
        g.bfs(r, out=out)
    g.profile(True, spans=True)
    t = 0.0
    k = 0.0
    spans = {}
    for r in roots:
        g.bfs(r, out=out)
        t += g.last_stats["device_ms"]
        k += g.last_stats["kernel_ms"]
        for kk, vv in g.profile_spans().items():
            spans[kk] = spans.get(kk, 0.0) + vv / len(roots)
    g.profile(False)
    t2 = 0.0
    for r in roots:
        g.bfs(r, out=out)
        t2 += g.last_stats["device_ms"]
    arcs = g.last_stats["arcs_decoded"]
    print(f"{tune:45s} bfs {t2 / len(roots):7.3f} ms (profiled {t / len(roots):7.3f})  expand {k / len(roots):7.3f} ms"
          f"  spans {{{', '.join(f'{a}: {b:.2f}' for a, b in spans.items())}}}", flush=True)
    g.unload()
