"""Full-size parity at BASELINE.json's configs[1..3] (C2 uk-2002-like, C3 twitter-like, C4 uk-2007-like), in the
launch configuration bench.py times (torch stream, in-CGR = the encoded transpose, direction-optimizing BFS).

Per config:
  * the product encoder's CGR bytes and bit offsets are identical to the oracle encoder's (SHA-256 of the bytes;
    the oracle's per-vertex-parallel encoder is pinned byte-identical to its serial one in test_oracle_codec.py);
  * BFS levels from 4 seeded roots are bit-exact against the oracle's BFS (OpenMP level-synchronous, pinned equal
    to the FIFO BFS in test_oracle_algos.py);
  * CC labels are bit-exact against the sequential union-find (C2, C4);
  * BC from 4 of the 64 seeded sources (C3) is within 1e-9 relative with exact zeros (Brandes, source-parallel,
    bit-identical to the serial oracle).
These generate the graphs at full size (C4: 105.9M vertices, 3.74B arcs; ~20 GB of host memory), so they run on
the GPU box only (-m gpu).
"""
import hashlib

import numpy as np
import pytest

import oracle as O
import paper_conf_sigmod_shalt19_b200 as G
import synth

pytestmark = [pytest.mark.gpu, pytest.mark.slow]


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    import torch
    if not torch.cuda.is_available():
        pytest.fail("no CUDA device (gpu tests must run on a B200)")
    torch.cuda.init()


def sha(a):
    return hashlib.sha256(np.ascontiguousarray(a).view(np.uint8)).hexdigest()


def check_bc(got, ref):
    got, ref = np.asarray(got), np.asarray(ref)
    assert np.array_equal(got == 0, ref == 0), "exact zeros must match"
    np.testing.assert_allclose(got, ref, rtol=1e-9, atol=0)


@pytest.mark.parametrize("name", ["c2", "c3", "c4"])
def test_full_size_config(name):
    import torch
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    P = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    cgr = G.encode(ro, co, *P)
    b, nb, offs, n, _ = cgr.view()
    ob, onb, ooffs = O.encode_par(ro, co, *P)
    assert nb == onb, (name, nb, onb)
    assert np.array_equal(offs, ooffs)
    assert sha(b) == sha(ob), name
    del ob, ooffs
    g = G.load(cgr, stream="torch", in_cgr=G.encode_transpose(ro, co, *P), symmetric=cfg.symmetric)
    lv = torch.empty(n, dtype=torch.int32, device="cuda")
    for r in synth.pick_roots(ro, 4):
        g.bfs(r, out=lv)
        assert np.array_equal(lv.cpu().numpy(), O.bfs_par(ro, co, r)), (name, r)
    if name in ("c2", "c4"):
        assert np.array_equal(g.cc(), O.cc(ro, co)), name
    if name == "c3":
        src = synth.bc_sources(ro, 64)[:4]
        check_bc(g.bc(src), O.bc_par(ro, co, src))
    g.unload()
