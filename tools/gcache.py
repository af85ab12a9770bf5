"""Per-call graph cache for the profiling tools (GPU box /tmp, same gpurun call only): the config's CSR row offsets,
its CGR and the transpose's CGR are built once and reloaded by later tool invocations of the same script.
Not used by bench.py or the tests (they always build their inputs)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402

import paper_conf_sigmod_shalt19_b200 as G  # noqa: E402
import synth  # noqa: E402

DIR = os.environ.get("GCGT_TOOL_CACHE", "/tmp/gcgt_tool_cache")


def graph(name):
    """-> (cfg, ro, cgr, incgr or None)"""
    cfg = synth.CONFIGS[name]
    P = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    base = os.path.join(DIR, name)
    paths = [base + ".ro.npy", base + ".cgr"] + ([] if cfg.symmetric else [base + ".in.cgr"])
    if all(os.path.exists(p) for p in paths):
        ro = np.load(paths[0])
        return cfg, ro, G.open_cgr(paths[1]), None if cfg.symmetric else G.open_cgr(paths[2])
    ro, co = cfg.make()
    cgr = G.encode(ro, co, *P)
    incgr = None if cfg.symmetric else G.encode_transpose(ro, co, *P)
    try:
        os.makedirs(DIR, exist_ok=True)
        np.save(paths[0], ro)
        cgr.save(paths[1])
        if incgr is not None:
            incgr.save(paths[2])
    except OSError:
        pass
    return cfg, ro, cgr, incgr
