"""Times BFS under several GCGT_TUNE settings on one config (device ms per BFS, mean over roots).
Usage: python tools/micro.py CONFIG NROOTS TUNE1 [TUNE2 ...]   (TUNE '-' = defaults)"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

cfgname, nroots, tunes = sys.argv[1], int(sys.argv[2]), sys.argv[3:]
cfg = synth.CONFIGS[cfgname]
ro, co = cfg.make()
P = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
cgr = G.encode(ro, co, *P)
incgr = None if cfg.symmetric else G.encode_transpose(ro, co, *P)
roots = synth.pick_roots(ro, nroots)
out = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")
ref = None
for tune in tunes:
    os.environ["GCGT_TUNE"] = "" if tune == "-" else tune
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
    g.bfs(roots[0], out=out)
    ms, lv = [], []
    for r in roots:
        g.bfs(r, out=out)
        ms.append(g.last_stats["device_ms"])
        lv.append(g.last_stats["iterations"])
    chk = int(out.sum().item())
    ref = chk if ref is None else ref
    print(f"{cfgname:8s} {tune:40s} {sum(ms) / len(ms):8.3f} ms/BFS  levels {sum(lv) / len(lv):5.1f}  "
          f"min {min(ms):.3f}  {'ok' if chk == ref else 'MISMATCH'}", flush=True)
    g.unload()
