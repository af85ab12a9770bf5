"""Times BFS (graph mode, CUDA events) on one config for a list of GCGT_TUNE strings (knobs never change results;
each tune is also checked against the first tune's levels).
Usage: python tools/sweep_tunes.py CONFIG NROOTS TUNE [TUNE ...]"""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

cfgname, nroots, tunes = sys.argv[1], int(sys.argv[2]), sys.argv[3:] or [""]
t0 = time.time()
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import gcache  # noqa: E402
cfg, ro, cgr, incgr = gcache.graph(cfgname)
print(f"# {cfgname} n={ro.size - 1} m={int(ro[-1])} prep {time.time() - t0:.1f}s", flush=True)
roots = synth.pick_roots(ro, nroots)
n = ro.size - 1
out = torch.empty(n, dtype=torch.int32, device="cuda")
ref = {}
for tune in tunes:
    os.environ["GCGT_TUNE"] = tune
    g = G.load(cgr, stream="torch", in_cgr=incgr, symmetric=cfg.symmetric)
    g.bfs(roots[0], out=out)
    ms = []
    for r in roots:
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        g.bfs(r, out=out)
        e1.record()
        torch.cuda.synchronize()
        ms.append(e0.elapsed_time(e1))
        h = hash(out.cpu().numpy().tobytes())
        if r in ref:
            assert ref[r] == h, (tune, r)
        else:
            ref[r] = h
    g.unload()
    print(f"{tune or '(default)':48s} bfs {sum(ms) / len(ms):8.3f} ms  min {min(ms):8.3f}  "
          f"[{' '.join(f'{x:.2f}' for x in ms)}]", flush=True)
