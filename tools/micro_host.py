"""HBM-resident vs host-resident CGR (§8 f4) on one config: device ms per BFS over the same roots, levels compared
between the two.  Usage: python tools/micro_host.py CONFIG NROOTS [--json out.json]"""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
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
res = {"config": cfgname, "roots": len(roots), "cgr_mb": cgr.view()[1] / 8e6}
lv = {}
for host in (False, True):
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric, host_resident=host)
    g.bfs(roots[0], out=out)
    ms, sums = [], []
    for r in roots:
        g.bfs(r, out=out)
        ms.append(g.last_stats["device_ms"])
        sums.append(out.clone())
    lv[host] = sums
    g.unload()
    res["host_ms" if host else "hbm_ms"] = sum(ms) / len(ms)
res["identical"] = all(torch.equal(a, b) for a, b in zip(lv[False], lv[True]))
res["slowdown"] = res["host_ms"] / res["hbm_ms"]
print(json.dumps(res), flush=True)
if "--json" in sys.argv:
    with open(sys.argv[sys.argv.index("--json") + 1], "w") as f:
        json.dump(res, f)
