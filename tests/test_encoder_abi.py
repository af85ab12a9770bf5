"""Product host encoder (gcgt_encode, C-ABI) vs the oracle encoder: bit-exact CGR bytes and bit_offsets
(FORMAT.md), plus the boundary itself: the library loads and exports every symbol include/gcgt.h declares,
error codes, save/open.  CPU only (-m "not gpu")."""
import hashlib
import os
import re

import numpy as np
import pytest

import oracle as O
import paper_conf_sigmod_shalt19_b200 as G
import synth
from graphs import random_graph, csr_from_edges

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def test_header_symbols_exported():
    """Every function declared in include/gcgt.h is exported by libgcgt.so (and listed in the binding)."""
    hdr = open(os.path.join(ROOT, "include", "gcgt.h")).read()
    declared = set(re.findall(r"^\s*(?:gcgt_status|void|const char\*)\s+(gcgt_\w+)\s*\(", hdr, re.M))
    assert declared == set(G.ABI_SYMBOLS)
    L = G.lib()
    for sym in declared:
        assert hasattr(L, sym), sym
    assert "sm_100a" in G.version()


def _same(ro, co, ml, sl, k):
    ob, onb, ooffs = O.encode(ro, co, ml, sl, k)
    cg = G.encode(ro, co, ml, sl, k)
    pb, pnb, poffs, n, params = cg.view()
    assert params == (ml, sl, k) and n == ro.size - 1
    assert pnb == onb
    assert np.array_equal(poffs, ooffs)
    assert hashlib.sha256(pb.tobytes()).hexdigest() == hashlib.sha256(ob.tobytes()).hexdigest()


PARAMS = [(ml, sl, k) for k in (1, 2, 3, 4, 5) for ml in (0, 2, 3, 4, 10) for sl in (0, 4, 8, 32, 64, 128)]


@pytest.mark.parametrize("ml,sl,k", PARAMS)
def test_encoder_bit_exact_random(ml, sl, k):
    for seed, (n, m) in enumerate([(1, 0), (9, 30), (257, 3000), (1000, 20000)]):
        if m:
            ro, co = random_graph(n, m, seed=seed + 100 * k + sl)
        else:
            ro, co = np.zeros(2, np.uint64), np.zeros(0, np.uint32)
        _same(ro, co, ml, sl, k)


@pytest.mark.parametrize("name", ["c1", "web_s", "social_s", "rmat_s"])
def test_encoder_bit_exact_configs(name):
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    _same(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)


def test_encoder_hub_many_segments():
    """One vertex with 200k residuals (thousands of segments) and one with 50k short intervals."""
    n = 2_000_000
    rng = np.random.default_rng(5)
    hub = np.unique(rng.integers(0, n, size=200_000))
    itv = np.concatenate([np.arange(s, s + 5) for s in range(1000, 1000 + 50_000 * 7, 7)])
    src = np.concatenate([np.zeros(hub.size, np.int64), np.ones(itv.size, np.int64)])
    dst = np.concatenate([hub, itv])
    ro, co = csr_from_edges(n, src, dst)
    for ml, sl, k in [(4, 32, 3), (4, 8, 1), (0, 0, 2), (4, 0, 3)]:
        _same(ro, co, ml, sl, k)


def test_encoder_errors():
    ro = np.array([0, 2, 2], dtype=np.uint64)
    for cols, code in [([1, 1], G.EUNSORTED), ([1, 0], G.EUNSORTED), ([0, 5], G.ERANGE)]:
        with pytest.raises(G.GcgtError) as e:
            G.encode(ro, np.array(cols, np.uint32))
        assert e.value.status == code
    for ml, k in [(1, 3), (4, 0), (4, 6)]:
        with pytest.raises(G.GcgtError) as e:
            G.encode(ro, np.array([0, 1], np.uint32), ml, 32, k)
        assert e.value.status == G.EINVAL
    n = 1000
    with pytest.raises(G.GcgtError) as e:
        G.encode(np.array([0] + [3] * n, np.uint64), np.array([100, 500, 900], np.uint32), 4, 1, 1)
    assert e.value.status == G.ESEGLEN


def test_save_open_from_arrays(tmp_path):
    ro, co = random_graph(500, 4000, seed=3)
    cg = G.encode(ro, co, 4, 32, 3)
    b, nb, offs, n, params = cg.view()
    path = str(tmp_path / "g.cgr")
    cg.save(path)
    c2 = G.open_cgr(path)
    b2, nb2, offs2, n2, p2 = c2.view()
    assert (nb2, n2, p2) == (nb, n, params) and np.array_equal(b2, b) and np.array_equal(offs2, offs)
    c3 = G.from_arrays(b, nb, offs, *params)
    assert np.array_equal(c3.view()[0], b)
    bad = offs.copy()
    bad[-1] += 1
    with pytest.raises(G.GcgtError) as e:
        G.from_arrays(b, nb, bad, *params)
    assert e.value.status == G.EFORMAT
    # a file whose offsets decrease (corrupt table) is rejected like from_arrays rejects it
    import struct
    with open(path, "r+b") as f:
        f.seek(8 + 8 + 8 + 16 + 8 * 3)
        f.write(struct.pack("<Q", int(offs[5]) + 10_000_000))
    with pytest.raises(G.GcgtError) as e:
        G.open_cgr(path)
    assert e.value.status == G.EFORMAT
    cg.save(path)
    with open(path, "r+b") as f:  # n >= 2^32 in the header
        f.seek(8)
        f.write(struct.pack("<Q", 1 << 33))
    with pytest.raises(G.GcgtError) as e:
        G.open_cgr(path)
    assert e.value.status == G.EFORMAT
    with open(path, "r+b") as f:
        f.write(b"XXXX")
    with pytest.raises(G.GcgtError) as e:
        G.open_cgr(path)
    assert e.value.status == G.EFORMAT


def test_load_without_gpu_fails_loudly():
    """No CPU fallback: without a CUDA device gcgt_load reports ECUDA."""
    import torch
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    ro, co = random_graph(50, 200, seed=1)
    with pytest.raises(G.GcgtError) as e:
        G.load(G.encode(ro, co))
    assert e.value.status == G.ECUDA


def _transpose(ro, co):
    n = ro.size - 1
    src = np.repeat(np.arange(n, dtype=np.int64), np.diff(ro.astype(np.int64)))
    from graphs import csr_from_edges
    return csr_from_edges(n, co.astype(np.int64), src)


@pytest.mark.parametrize("ml,sl,k", [(4, 32, 3), (0, 0, 1), (2, 8, 2)])
def test_encode_transpose_bit_exact(ml, sl, k):
    """gcgt_encode_transpose(G) == oracle encode of the transposed CSR (in-arcs, rows sorted)."""
    ro, co = random_graph(800, 9000, seed=k + sl)
    tro, tco = _transpose(ro, co)
    ob, onb, ooffs = O.encode(tro, tco, ml, sl, k)
    b, nb, offs, n, _ = G.encode_transpose(ro, co, ml, sl, k).view()
    assert nb == onb and np.array_equal(offs, ooffs) and np.array_equal(b, ob)


def test_load_csr_validates_then_fails_loudly_without_gpu():
    """The CSR baseline checks its input before touching the device (ERANGE for an id >= n), and has no CPU
    fallback either (ECUDA without a device)."""
    import torch
    ro, co = random_graph(50, 200, seed=2)
    bad = co.copy()
    bad[3] = 50
    with pytest.raises(G.GcgtError) as e:
        G.load_csr(ro, bad)
    assert e.value.status == G.ERANGE
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    with pytest.raises(G.GcgtError) as e:
        G.load_csr(ro, co)
    assert e.value.status == G.ECUDA


@pytest.mark.parametrize("scale,parts", [(12, 3), (20, 4)])
def test_rmat_slices_encode_like_the_whole_graph(scale, parts):
    """C5's pipeline (§8(d) C5: R-MAT s29 cannot be held as one CSR): each vertex-range slice is generated alone
    (synth.rmat_slice) and encoded alone (gcgt_encode_slice); the slices' CGRs concatenated are byte-identical to
    the oracle's encoding of the whole graph, and each slice equals the whole CGR's bits of its range."""
    import synth
    ro, co = synth.rmat(scale, 16, 29)
    n = ro.size - 1
    b = synth.rmat_slices(scale, 16, 29, parts)
    slices = []
    for r in range(parts):
        sro, sco = synth.rmat_slice(scale, 16, 29, b[r], b[r + 1])
        s = G.encode_slice(sro, sco, b[r], n, 4, 32, 3)
        assert G.slice_info(s) == (b[r], n)
        slices.append(s)
    whole = G.concat(slices)
    wb, wnb, woffs, wn, _ = whole.view()
    ob, onb, ooffs = O.encode_par(ro, co, 4, 32, 3)
    assert (wn, wnb) == (n, onb) and np.array_equal(woffs, ooffs) and np.array_equal(wb, ob)
    bits = np.unpackbits(ob)
    for r, s in enumerate(slices):  # each slice = the whole stream's bits [offs[lo], offs[hi]), offsets re-based
        sb, snb, soffs, sn, _ = s.view()
        lo, hi = b[r], b[r + 1]
        assert sn == hi - lo and np.array_equal(soffs, ooffs[lo:hi + 1] - ooffs[lo])
        assert np.array_equal(np.unpackbits(sb)[:snb], bits[int(ooffs[lo]):int(ooffs[hi])])
    with pytest.raises(G.GcgtError) as e:  # not consecutive
        G.concat([slices[0], slices[-1]])
    assert e.value.status == G.EINVAL
