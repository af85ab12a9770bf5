"""GPU parity: the sm_100a path (through the C ABI) vs the oracle, element by element (-m gpu).

BFS levels and CC labels are bit-exact; BC within 1e-9 relative with exact zeros (north_star tolerance; the two
sides differ only in fp64 summation order).  Inputs: seeded synthetic graphs of each recipe at sizes
the oracle finishes in seconds (several tiles and a ragged tail), every (zeta_k, segmented) kernel instantiation,
and the degenerate cases.
"""
import numpy as np
import pytest

import oracle as O
import paper_conf_sigmod_shalt19_b200 as G
import synth
from graphs import random_graph, csr_from_edges

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    import torch
    if not torch.cuda.is_available():
        pytest.fail("no CUDA device (gpu tests must run on a B200)")
    torch.cuda.init()


def load(ro, co, ml=4, sl=32, k=3):
    return G.load(G.encode(ro, co, ml, sl, k))


def check_bc(got, ref):
    got, ref = np.asarray(got), np.asarray(ref)
    assert np.array_equal(got == 0, ref == 0), "exact zeros must match"
    np.testing.assert_allclose(got, ref, rtol=1e-9, atol=0)


PARAMS = [(ml, sl, k) for k in (1, 2, 3, 4, 5) for (ml, sl) in ((4, 32), (0, 0), (2, 8), (4, 0), (3, 64))]


@pytest.mark.parametrize("ml,sl,k", PARAMS)
def test_bfs_cc_random_all_instantiations(ml, sl, k):
    for seed, (n, m, sym) in enumerate([(1, 0, False), (33, 100, True), (5000, 60000, False), (20000, 300000, True)]):
        if m:
            ro, co = random_graph(n, m, seed=seed + 7 * k, symmetric=sym)
        else:
            ro, co = np.zeros(n + 1, np.uint64), np.zeros(0, np.uint32)
        g = load(ro, co, ml, sl, k)
        for s in sorted({0, n // 3, n - 1}):
            assert np.array_equal(g.bfs(s), O.bfs(ro, co, s)), (seed, s)
        assert np.array_equal(g.cc(), O.cc(ro, co)), seed


@pytest.mark.parametrize("name", ["c1", "web_s", "social_s", "rmat_s"])
def test_bfs_configs(name):
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    g = load(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    roots = [0] + synth.pick_roots(ro, 4)
    deg = np.diff(ro.astype(np.int64))
    for r in roots:
        lv = g.bfs(r)
        ref = O.bfs(ro, co, r)
        assert np.array_equal(lv, ref), r
        assert g.last_stats["arcs_decoded"] == int(deg[ref >= 0].sum())
        assert g.last_stats["vertices_expanded"] == int((ref >= 0).sum())


@pytest.mark.parametrize("name", ["c1", "web_s", "social_s", "rmat_s"])
def test_cc_configs(name):
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    g = load(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    assert np.array_equal(g.cc(), O.cc(ro, co))


@pytest.mark.parametrize("name,nsrc", [("c1", 64), ("web_s", 4), ("social_s", 3), ("rmat_s", 3)])
def test_bc_configs(name, nsrc):
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    g = load(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    src = synth.bc_sources(ro, nsrc)
    check_bc(g.bc(src), O.bc(ro, co, src))


@pytest.mark.parametrize("ml,sl,k", [(4, 32, 3), (0, 0, 1), (2, 8, 2), (4, 0, 5)])
def test_bc_random(ml, sl, k):
    for seed, (n, m) in enumerate([(2, 1), (12, 30), (700, 5000)]):
        ro, co = random_graph(n, m, seed=seed + k, symmetric=bool(seed % 2))
        g = load(ro, co, ml, sl, k)
        src = list(range(n)) if n <= 12 else [0, 5, 5, n - 1]
        check_bc(g.bc(src), O.bc(ro, co, src))


def test_degenerate_cases():
    # isolated source, self-loops, empty graph, source with only a self-loop
    n = 100
    ro, co = csr_from_edges(n, [3, 3, 5, 7, 7], [3, 4, 5, 7, 8])
    g = load(ro, co)
    for s in (0, 3, 5, 7, 99):
        assert np.array_equal(g.bfs(s), O.bfs(ro, co, s))
    assert np.array_equal(g.cc(), O.cc(ro, co))
    check_bc(g.bc([0, 3, 5, 7]), O.bc(ro, co, [0, 3, 5, 7]))
    ro0, co0 = np.zeros(n + 1, np.uint64), np.zeros(0, np.uint32)
    g0 = load(ro0, co0)
    assert np.array_equal(g0.bfs(42), O.bfs(ro0, co0, 42))
    assert np.array_equal(g0.cc(), np.arange(n, dtype=np.uint32))
    with pytest.raises(G.GcgtError) as e:
        g0.bfs(n)
    assert e.value.status == G.ERANGE
    with pytest.raises(G.GcgtError) as e:
        g0.bc([n])
    assert e.value.status == G.ERANGE


def test_hub_and_long_intervals():
    """A hub with 300k residuals (thousands of segments), a vertex with 20k short intervals, one with a 1M-long
    interval crossing many bitmap words, and ids near n."""
    n = 3_000_000
    rng = np.random.default_rng(11)
    hub = np.unique(rng.integers(0, n, size=300_000))
    itv = np.concatenate([np.arange(s, s + 6) for s in range(5, 5 + 20_000 * 9, 9)])
    long_run = np.arange(1_500_000, 2_500_000)
    tail = np.arange(n - 40, n)
    src = np.concatenate([np.zeros(hub.size), np.ones(itv.size), np.full(long_run.size, 2),
                          np.full(tail.size, 3), [hub[5]] * 3]).astype(np.int64)
    dst = np.concatenate([hub, itv, long_run, tail, [1, 2, 3]]).astype(np.int64)
    ro, co = csr_from_edges(n, src, dst)
    for ml, sl, k in [(4, 32, 3), (4, 8, 1), (0, 0, 3), (2, 128, 2), (4, 0, 1)]:
        g = load(ro, co, ml, sl, k)
        for s in (0, 1, 2, 3):
            assert np.array_equal(g.bfs(s), O.bfs(ro, co, s)), (ml, sl, k, s)
        assert np.array_equal(g.cc(), O.cc(ro, co))
        check_bc(g.bc([0, 1]), O.bc(ro, co, [0, 1]))


def test_device_outputs_torch():
    import torch
    ro, co = synth.CONFIGS["c1"].make()
    g = G.load(G.encode(ro, co, 4, 64, 3), stream="torch")
    out = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")
    g.bfs(0, out=out)
    assert np.array_equal(out.cpu().numpy(), O.bfs(ro, co, 0))
    lab = torch.empty(ro.size - 1, dtype=torch.int32, device="cuda")
    g.cc(out=lab)
    assert np.array_equal(lab.cpu().numpy().astype(np.uint32), O.cc(ro, co))
    bc = torch.empty(ro.size - 1, dtype=torch.float64, device="cuda")
    g.bc([0, 1, 2], out=bc)
    check_bc(bc.cpu().numpy(), O.bc(ro, co, [0, 1, 2]))


def test_c1_baseline_config_exact():
    """BASELINE.json configs[0]: BFS from vertex 0 on R-MAT s10 ef16, minLen 4, segment 64 B."""
    ro, co = synth.CONFIGS["c1"].make()
    g = load(ro, co, 4, 64, 3)
    assert np.array_equal(g.bfs(0), O.bfs(ro, co, 0))


@pytest.mark.slow
def test_c2_full_size_bench_launch():
    """configs[1] at full size in the bench's launch configuration: BFS from the bench roots, all levels compared
    with the oracle (CSR BFS, seconds in C); CC labels compared too."""
    cfg = synth.CONFIGS["c2"]
    ro, co = cfg.make()
    g = G.load(G.encode(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k), stream="torch")
    for r in synth.pick_roots(ro, 2):
        assert np.array_equal(g.bfs(r), O.bfs(ro, co, r)), r
    assert np.array_equal(g.cc(), O.cc(ro, co))


# ---------------------------------------------------------------------------------------------------------------------
# The device warp decoder (Alg. 4 analogue) pinned against the paper's Fig. 5 and against serial decoding
# ---------------------------------------------------------------------------------------------------------------------
def test_warp_decoder_fig5_trace(golden):
    """Fig. 5: 16 threads, gamma, bit array of 1..5.  The device trace must reproduce every
    printed poss / flags row and the decoded values 1..5."""
    g = golden("fig5.txt")
    b, nb = O.bits_to_bytes(g["bits"][0])
    vals, tpos, tflags, rounds = G.debug_warp_decode(b, nb, 1, 16, 5)
    assert list(vals) == [1, 2, 3, 4, 5]
    assert rounds == 4
    X = 0xFFFFFFFF
    for r in range(4):
        exp = [X if t == "x" else int(t) for t in g[f"poss{r}"]]
        assert [int(x) for x in tpos[r]] == exp, r
        assert [int(x) for x in tflags[r]] == [int(t) for t in g[f"flags{r}"]], r


@pytest.mark.parametrize("k", [1, 2, 3, 4, 5])
def test_warp_decoder_random_streams(k):
    rng = np.random.default_rng(77 + k)
    for trial in range(6):
        hi = [2, 8, 1 << 10, 1 << 20, 1 << 33, 1 << 40][trial]
        xs = [int(x) for x in rng.integers(1, hi, size=500)]
        bits = "".join(O.vlc_string(k, x) for x in xs)
        b, nb = O.bits_to_bytes(bits)
        vals, _, _, _ = G.debug_warp_decode(b, nb, k, 32, len(xs))
        assert [int(v) for v in vals] == xs, (k, trial)


# ---------------------------------------------------------------------------------------------------------------------
# Direction-optimizing BFS (bottom-up levels over the in-CGR, §8 a9)
# ---------------------------------------------------------------------------------------------------------------------
@pytest.mark.parametrize("tune", ["", "bu_alpha=100000,bu_beta=1", "bu_alpha=100000,bu_beta=100000", "graph=0",
                                  "graph=0,bu_alpha=100000,bu_beta=1", "graph=0,chunk=2", "graph=0,chunk=16",
                                  "hub_segs=1", "compact=0", "dir_bits=1", "dir_opt=0", "bu_alpha=1", "td_stage=0",
                                  "td_pool=1", "td_pool=1,td_stage=0", "ck_c=2", "ck_c=1", "ck_c=32",
                                  "ck_c=0", "bu_grow=0,bu_alpha=25", "hub_stage=0", "td_pool=0",
                                  "td_pool=0,bu_alpha=100000,bu_beta=1", "ck_c=4", "ck_c=3,td_pool=0", "dir_edges=0",
                                  "edge_guard=10,alpha_edges2=1000", "alpha_edges=140",
                                  "dir_edges=1", "dir_edges=1,alpha_edges=10", "dir_edges=1,alpha_edges=1000"])
@pytest.mark.parametrize("name", ["c1", "rmat_s", "web_s", "social_s"])
def test_bfs_direction_optimizing(name, tune, monkeypatch):
    """Symmetric graphs use the out-CGR as in-CGR; directed ones the encoded transpose.  The tunes force
    bottom-up early (and keep it), or switch back and forth, so every level kind is exercised."""
    monkeypatch.setenv("GCGT_TUNE", tune)
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    p = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    cgr = G.encode(ro, co, *p)
    if cfg.symmetric:
        g = G.load(cgr, symmetric=True)
    else:
        g = G.load(cgr, in_cgr=G.encode_transpose(ro, co, *p))
    for r in [0] + synth.pick_roots(ro, 3):
        assert np.array_equal(g.bfs(r), O.bfs(ro, co, r)), (name, tune, r)


@pytest.mark.parametrize("tune", ["td_pool=1", "td_pool=0", "td_stage=0", "hub_segs=1", "ck_c=2", "ck_c=0", "ck_c=32",
                                  "td_pool=0,hub_segs=8"])
@pytest.mark.parametrize("name", ["web_s", "social_s", "rmat_s"])
def test_cc_bc_engine_knobs(name, tune, monkeypatch):
    """CC hooking and BC run through the same expansion engine: every engine knob keeps them exact."""
    monkeypatch.setenv("GCGT_TUNE", tune)
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    g = load(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    assert np.array_equal(g.cc(), O.cc(ro, co))
    src = synth.bc_sources(ro, 2)
    check_bc(g.bc(src), O.bc(ro, co, src))


@pytest.mark.parametrize("ml,sl,k", [(4, 32, 3), (0, 0, 1), (2, 8, 5)])
def test_bfs_bottom_up_random(ml, sl, k, monkeypatch):
    monkeypatch.setenv("GCGT_TUNE", "bu_alpha=100000,bu_beta=1")
    for seed, sym in [(1, True), (2, False), (3, False)]:
        ro, co = random_graph(6000, 60000, seed=seed + k, symmetric=sym)
        cgr = G.encode(ro, co, ml, sl, k)
        g = G.load(cgr, symmetric=True) if sym else G.load(cgr, in_cgr=G.encode_transpose(ro, co, ml, sl, k))
        for s in (0, 17, 5999):
            assert np.array_equal(g.bfs(s), O.bfs(ro, co, s)), (seed, s)


# ---------------------------------------------------------------------------------------------------------------------
# Uncompressed-CSR baseline (§8 f3): same levels as the oracle on every recipe, top-down and direction-optimizing
# ---------------------------------------------------------------------------------------------------------------------
@pytest.mark.parametrize("tune", ["", "bu_alpha=100000,bu_beta=1", "bu_alpha=100000,bu_beta=100000"])
@pytest.mark.parametrize("name", ["c1", "rmat_s", "web_s", "social_s"])
def test_csr_baseline_bfs(name, tune, monkeypatch):
    monkeypatch.setenv("GCGT_TUNE", tune)
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    for dopt in (False, True):
        g = G.load_csr(ro, co, symmetric=cfg.symmetric, direction_optimizing=dopt)
        for r in [0] + synth.pick_roots(ro, 3):
            assert np.array_equal(g.bfs(r), O.bfs(ro, co, r)), (name, tune, dopt, r)
        g.unload()


def test_csr_baseline_hubs_and_errors():
    """Hub vertices (more than kCsrHub = 4096 arcs: chunked over the grid), isolated vertices, and the BFS-only
    contract (CC / BC refuse a CSR graph)."""
    n = 200_000
    rng = np.random.default_rng(5)
    hub = np.unique(rng.integers(0, n, size=50_000))
    src = np.concatenate([np.zeros(hub.size), rng.integers(0, n, size=100_000)]).astype(np.int64)
    dst = np.concatenate([hub, rng.integers(0, n, size=100_000)]).astype(np.int64)
    ro, co = csr_from_edges(n, src, dst)
    g = G.load_csr(ro, co, direction_optimizing=True)
    for s in (0, 1, int(hub[3]), n - 1):
        assert np.array_equal(g.bfs(s), O.bfs(ro, co, s)), s
    with pytest.raises(G.GcgtError) as e:
        g.cc()
    assert e.value.status == G.EINVAL
    with pytest.raises(G.GcgtError) as e:
        g.bc([0])
    assert e.value.status == G.EINVAL


# ---------------------------------------------------------------------------------------------------------------------
# Host-resident CGR (§8 f4): the kernels decode from pinned, mapped host memory; results identical to the oracle
# ---------------------------------------------------------------------------------------------------------------------
@pytest.mark.parametrize("name", ["c1", "web_s", "social_s", "rmat_s"])
def test_host_resident_cgr(name):
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    p = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    cgr = G.encode(ro, co, *p)
    inc = None if cfg.symmetric else G.encode_transpose(ro, co, *p)
    g = G.load(cgr, in_cgr=inc, symmetric=cfg.symmetric, host_resident=True)
    for r in [0] + synth.pick_roots(ro, 3):
        assert np.array_equal(g.bfs(r), O.bfs(ro, co, r)), (name, r)
    assert np.array_equal(g.cc(), O.cc(ro, co)), name
    src = synth.pick_roots(ro, 2)
    check_bc(g.bc(src), O.bc(ro, co, src))
    g.unload()


# ---------------------------------------------------------------------------------------------------------------------
# Repeated loads of a pinned CGR (gcgt_cgr_pin: derived load tables cached with the CGR, host arrays page-locked)
# ---------------------------------------------------------------------------------------------------------------------
@pytest.mark.parametrize("tune", ["", "ck_c=2", "compact=0"])
@pytest.mark.parametrize("name", ["web_s", "social_s"])
def test_pinned_cgr_reload(name, tune, monkeypatch):
    monkeypatch.setenv("GCGT_TUNE", tune)
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    p = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    cgr, incgr = G.encode(ro, co, *p), G.encode_transpose(ro, co, *p)
    roots = synth.pick_roots(ro, 2)
    for it in range(3):  # before pinning (tables built by the load), pinned, pinned again (cached tables)
        if it == 1:
            cgr.pin()
            incgr.pin()
        g = G.load(cgr, in_cgr=incgr)
        for r in roots:
            assert np.array_equal(g.bfs(r), O.bfs(ro, co, r)), (name, tune, it, r)
        g.unload()
