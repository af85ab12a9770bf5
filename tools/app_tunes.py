"""Times CC or BC (device ms per call, from the library's CUDA events) on one config for a list of GCGT_TUNE strings;
every tune's output is checked against the first tune's.
Usage: python tools/app_tunes.py cc|bc CONFIG N TUNE [TUNE ...]   (N = repetitions for CC, sources for BC)"""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import gcache  # noqa: E402
import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

app, cfgname, N, tunes = sys.argv[1], sys.argv[2], int(sys.argv[3]), sys.argv[4:] or [""]
t0 = time.time()
cfg, ro, cgr, incgr = gcache.graph(cfgname)
n = ro.size - 1
print(f"# {app} {cfgname} n={n} m={int(ro[-1])} prep {time.time() - t0:.1f}s", flush=True)
ref = None
for tune in tunes:
    os.environ["GCGT_TUNE"] = tune
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
    if app == "cc":
        out = torch.empty(n, dtype=torch.int32, device="cuda")
        g.cc(out=out)
        ms = []
        for _ in range(N):
            g.cc(out=out)
            ms.append(g.last_stats["device_ms"])
        res = out.cpu().numpy()
    else:
        src = synth.bc_sources(ro, N)
        res = g.bc(src)
        ms = [g.last_stats["device_ms"] / N]
    if ref is None:
        ref = res
    elif app == "cc":
        assert np.array_equal(ref, res), tune
    else:
        assert np.allclose(ref, res, rtol=1e-9, atol=0), tune
    g.unload()
    print(f"{tune or '(default)':48s} {app} {np.median(ms):9.3f} ms{' per source' if app == 'bc' else ''}", flush=True)
