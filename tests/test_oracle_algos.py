"""Pins for the oracle's BFS / CC / BC (-m "not gpu").

BFS: Fig. 1 levels, Bellman-Ford fixpoint (a different algorithm) on random graphs, BFS over the decoded CGR.
CC: brute-force reachability on the undirected closure, Fig. 1.
BC: the definition bc(v) = sum_{s in S, t != s, v} sigma_st(v)/sigma_st computed from all-pairs path counts
(not Brandes' recursion), closed forms (path, star, cycle, complete graph), and the checksum
sum_v bc(v) = sum_{s in S} sum_{t reached, t != s} (d(s,t) - 1).
"""
import itertools

import numpy as np
import pytest

import oracle as O
from graphs import csr_from_edges, random_graph, adjacency_lists


def fig1(golden):
    g = golden("fig1.txt")
    return (np.array([int(v) for v in g["row_offsets"]], dtype=np.uint64),
            np.array([int(v) for v in g["cols"]], dtype=np.uint32), g)


def test_fig1_bfs_cc(golden):
    ro, co, g = fig1(golden)
    assert list(O.bfs(ro, co, 0)) == [int(v) for v in g["bfs0"]]
    assert list(O.cc(ro, co)) == [int(v) for v in g["cc"]]


def bellman_ford_levels(n, adj, s):
    INF = 1 << 60
    d = [INF] * n
    d[s] = 0
    changed = True
    while changed:
        changed = False
        for u in range(n):
            if d[u] < INF:
                for v in adj[u]:
                    if d[u] + 1 < d[v]:
                        d[v] = d[u] + 1
                        changed = True
    return [x if x < INF else -1 for x in d]


@pytest.mark.parametrize("seed", range(12))
def test_bfs_vs_bellman_ford(seed):
    n = [1, 2, 5, 17, 40, 64][seed % 6]
    ro, co = random_graph(n, 3 * n, seed=seed, symmetric=seed % 2 == 0)
    adj = adjacency_lists(ro, co)
    for s in range(0, n, max(1, n // 4)):
        assert list(O.bfs(ro, co, s)) == bellman_ford_levels(n, adj, s)


@pytest.mark.parametrize("ml,sl,k", [(4, 32, 3), (0, 0, 1), (2, 8, 2), (4, 0, 3)])
def test_bfs_on_cgr_equals_bfs(ml, sl, k):
    ro, co = random_graph(500, 5000, seed=ml + sl + k)
    b, nb, offs = O.encode(ro, co, ml, sl, k)
    for s in (0, 17, 499):
        lv, edges = O.bfs_cgr(b, offs, ml, sl, k, s)
        ref = O.bfs(ro, co, s)
        assert np.array_equal(lv, ref)
        deg = np.diff(ro.astype(np.int64))
        assert edges == int(deg[ref >= 0].sum())


@pytest.mark.parametrize("threads", [1, 2, 3, 8])
def test_bfs_par_equals_bfs(threads):
    """The OpenMP level-synchronous BFS (gcgt_oracle_par.c) gives the FIFO BFS's unique levels,
    over the CSR and over the oracle's own CGR, with the edge count of the reached vertices."""
    for seed, (n, m, sym) in enumerate([(1, 0, False), (64, 200, True), (3000, 30000, False), (20000, 250000, True)]):
        if m:
            ro, co = random_graph(n, m, seed=seed + 31 * threads, symmetric=sym)
        else:
            ro, co = np.zeros(n + 1, np.uint64), np.zeros(0, np.uint32)
        deg = np.diff(ro.astype(np.int64))
        for ml, sl, k in [(4, 32, 3), (0, 0, 1), (2, 8, 5)]:
            b, nb, offs = O.encode(ro, co, ml, sl, k)
            for s in sorted({0, n // 2, n - 1}):
                ref = O.bfs(ro, co, s)
                assert np.array_equal(O.bfs_par(ro, co, s, threads), ref), (seed, s)
                lv, edges = O.bfs_cgr_par(b, offs, ml, sl, k, s, threads)
                assert np.array_equal(lv, ref), (seed, ml, sl, k, s)
                assert edges == int(deg[ref >= 0].sum())


@pytest.mark.parametrize("name", ["c1", "web_s", "social_s", "rmat_s"])
def test_bfs_par_on_recipes(name):
    import synth
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    b, nb, offs = O.encode(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    for r in [0] + synth.pick_roots(ro, 2):
        ref = O.bfs(ro, co, r)
        assert np.array_equal(O.bfs_par(ro, co, r), ref)
        lv, _ = O.bfs_cgr_par(b, offs, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k, r)
        assert np.array_equal(lv, ref)


@pytest.mark.parametrize("threads", [1, 3, 8])
def test_bc_par_bit_identical(threads):
    """orc_bc_par sums the per-source dependency vectors in source order: bit-identical to orc_bc."""
    for seed, (n, m, sym) in enumerate([(12, 30, False), (700, 5000, True), (3000, 20000, False)]):
        ro, co = random_graph(n, m, seed=seed + threads, symmetric=sym)
        src = [0, 5, 5, n - 1, 3, 1, 7, 2, 9, 11][: 4 + seed * 3]
        assert np.array_equal(O.bc_par(ro, co, src, threads), O.bc(ro, co, src))


def brute_cc(n, adj):
    und = [set() for _ in range(n)]
    for u in range(n):
        for v in adj[u]:
            und[u].add(v)
            und[v].add(u)
    lab = [-1] * n
    for s in range(n):  # s ascending: the first vertex to reach a component is its minimum id
        if lab[s] >= 0:
            continue
        stack = [s]
        lab[s] = s
        while stack:
            x = stack.pop()
            for y in und[x]:
                if lab[y] < 0:
                    lab[y] = s
                    stack.append(y)
    return lab


@pytest.mark.parametrize("seed", range(10))
def test_cc_vs_brute_force(seed):
    n = [1, 3, 10, 50, 200][seed % 5]
    ro, co = random_graph(n, n // 2 + 1, seed=seed, locality=0.3)
    lab = O.cc(ro, co)
    assert list(lab) == brute_cc(n, adjacency_lists(ro, co))
    # invariants: lab[v] <= v, lab[lab[v]] == lab[v], endpoints of every arc agree
    for u, lst in enumerate(adjacency_lists(ro, co)):
        assert lab[u] <= u and lab[lab[u]] == lab[u]
        for v in lst:
            assert lab[u] == lab[v]


def test_cc_exhaustive_n4():
    """Every digraph on 4 vertices (2^12 arc sets)."""
    n = 4
    pairs = [(a, b) for a in range(n) for b in range(n) if a != b]
    for mask in range(1 << len(pairs)):
        src = [p[0] for i, p in enumerate(pairs) if mask >> i & 1]
        dst = [p[1] for i, p in enumerate(pairs) if mask >> i & 1]
        ro, co = csr_from_edges(n, src, dst)
        assert list(O.cc(ro, co)) == brute_cc(n, adjacency_lists(ro, co))


# ---------------------------------------------------------------------------------------------------------------
# BC
# ---------------------------------------------------------------------------------------------------------------
def all_pairs_counts(n, adj):
    """dist[s][t], sigma[s][t] by BFS counting from every s."""
    dist = [[-1] * n for _ in range(n)]
    sig = [[0] * n for _ in range(n)]
    for s in range(n):
        dist[s][s] = 0
        sig[s][s] = 1
        frontier = [s]
        while frontier:
            nxt = []
            for u in frontier:
                for v in adj[u]:
                    if dist[s][v] < 0:
                        dist[s][v] = dist[s][u] + 1
                        nxt.append(v)
            for u in frontier:
                for v in adj[u]:
                    if dist[s][v] == dist[s][u] + 1:
                        sig[s][v] += sig[s][u]
            frontier = sorted(set(nxt))
    return dist, sig


def bc_definition(n, adj, sources):
    """bc(v) = sum_{s in S} sum_{t != s, t != v} sigma_st(v) / sigma_st, sigma_st(v) = sigma_sv sigma_vt when
    d(s,v) + d(v,t) = d(s,t) (the definition; exact rational arithmetic via Python ints)."""
    from fractions import Fraction
    dist, sig = all_pairs_counts(n, adj)
    bc = [Fraction(0)] * n
    for s in sources:
        for t in range(n):
            if t == s or dist[s][t] < 0:
                continue
            for v in range(n):
                if v in (s, t) or dist[s][v] < 0 or dist[v][t] < 0:
                    continue
                if dist[s][v] + dist[v][t] == dist[s][t]:
                    bc[v] += Fraction(sig[s][v] * sig[v][t], sig[s][t])
    return [float(x) for x in bc]


@pytest.mark.parametrize("seed", range(16))
def test_bc_vs_definition(seed):
    rng = np.random.default_rng(seed)
    n = int(rng.integers(2, 13))
    m = int(rng.integers(1, 3 * n))
    ro, co = random_graph(n, m, seed=seed, symmetric=bool(seed % 2), locality=0.4)
    adj = adjacency_lists(ro, co)
    sources = list(range(n)) if seed % 3 else [int(x) for x in rng.integers(0, n, size=5)]  # duplicates allowed
    got = O.bc(ro, co, sources)
    ref = bc_definition(n, adj, sources)
    np.testing.assert_allclose(got, ref, rtol=1e-12, atol=0)


def test_bc_exhaustive_n4():
    n = 4
    pairs = [(a, b) for a in range(n) for b in range(n) if a != b]
    rng = np.random.default_rng(4)
    for mask in rng.choice(1 << len(pairs), size=300, replace=False):
        src = [p[0] for i, p in enumerate(pairs) if int(mask) >> i & 1]
        dst = [p[1] for i, p in enumerate(pairs) if int(mask) >> i & 1]
        ro, co = csr_from_edges(n, src, dst)
        np.testing.assert_allclose(O.bc(ro, co, list(range(n))), bc_definition(n, adjacency_lists(ro, co),
                                                                             list(range(n))), rtol=1e-12)


def _path(n, symmetric):
    return csr_from_edges(n, list(range(n - 1)), list(range(1, n)), symmetric=symmetric)


@pytest.mark.parametrize("n", [2, 3, 6, 11])
def test_bc_closed_forms(n):
    allsrc = list(range(n))
    # symmetric path P_n: bc[i] = 2 i (n-1-i)
    ro, co = _path(n, True)
    assert list(O.bc(ro, co, allsrc)) == [2.0 * i * (n - 1 - i) for i in range(n)]
    # directed path: i (n-1-i)
    ro, co = _path(n, False)
    assert list(O.bc(ro, co, allsrc)) == [1.0 * i * (n - 1 - i) for i in range(n)]
    # star (symmetric): centre (n-1)(n-2), leaves 0
    ro, co = csr_from_edges(n, [0] * (n - 1), list(range(1, n)), symmetric=True)
    assert list(O.bc(ro, co, allsrc)) == [float((n - 1) * (n - 2))] + [0.0] * (n - 1)
    # complete graph: 0
    src, dst = zip(*[(a, b) for a in range(n) for b in range(n) if a != b])
    ro, co = csr_from_edges(n, src, dst)
    assert list(O.bc(ro, co, allsrc)) == [0.0] * n


@pytest.mark.parametrize("n", [3, 5, 7, 9, 13])
def test_bc_odd_cycle(n):
    ro, co = csr_from_edges(n, list(range(n)), [(i + 1) % n for i in range(n)], symmetric=True)
    assert list(O.bc(ro, co, list(range(n)))) == [(n - 1) * (n - 3) / 4.0] * n


@pytest.mark.parametrize("seed", range(4))
def test_bc_checksum(seed):
    """sum_v bc(v) = sum_{s in S} sum_{t reached, t != s} (d(s,t) - 1): every shortest s-t path has d-1 interior
    vertices, and the pair's dependency is split over paths with weights summing to 1."""
    ro, co = random_graph(300, 2000, seed=seed)
    rng = np.random.default_rng(seed)
    S = [int(x) for x in rng.integers(0, 300, size=8)]
    got = O.bc(ro, co, S).sum()
    ref = 0
    for s in S:
        lv = O.bfs(ro, co, s)
        ref += int((lv[lv > 0] - 1).sum())
    assert got == pytest.approx(ref, rel=1e-12)


def test_bfs_cgr_sample_counts_whole_levels():
    """The timing sample expands whole BFS levels until the arc budget is met: its arc count is the out-degree sum
    of the vertices of the first L levels (for some L), at least the budget unless the BFS ran out."""
    ro, co = random_graph(5000, 60000, seed=4)
    b, nb, offs = O.encode(ro, co, 4, 32, 3)
    ref = O.bfs(ro, co, 0)
    deg = np.diff(ro.astype(np.int64))
    per_level = [int(deg[ref == d].sum()) for d in range(ref.max() + 1)]
    prefix = np.cumsum(per_level)
    for budget in (1, 500, 5000, 20000, 10**12):
        e = O.bfs_cgr_sample(b, offs, 4, 32, 3, 0, budget, 3)
        assert e in set(prefix.tolist())
        assert e >= budget or e == prefix[-1]
