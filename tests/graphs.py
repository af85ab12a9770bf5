"""Small seeded graph builders for the CPU tests (pure numpy; no method arithmetic)."""
import numpy as np


def csr_from_edges(n, src, dst, symmetric=False, drop_self=False):
    src = np.asarray(src, dtype=np.int64)
    dst = np.asarray(dst, dtype=np.int64)
    if symmetric:
        src, dst = np.concatenate([src, dst]), np.concatenate([dst, src])
    if drop_self:
        keep = src != dst
        src, dst = src[keep], dst[keep]
    key = np.unique(src * n + dst) if src.size else np.zeros(0, dtype=np.int64)
    s, d = key // n, key % n
    rowoff = np.zeros(n + 1, dtype=np.uint64)
    np.add.at(rowoff, s + 1, 1)
    rowoff = np.cumsum(rowoff).astype(np.uint64)
    return rowoff, d.astype(np.uint32)


def random_graph(n, m, seed, symmetric=False, locality=0.5):
    """Random digraph with a mix of local runs (intervals) and random arcs (residuals)."""
    rng = np.random.default_rng(seed)
    src = rng.integers(0, n, size=m)
    far = rng.integers(0, n, size=m)
    near = np.clip(src + rng.integers(-8, 9, size=m), 0, n - 1)
    dst = np.where(rng.random(m) < locality, near, far)
    # runs: some vertices get a consecutive block
    nb = max(1, m // 16)
    bu = rng.integers(0, n, size=nb)
    bs = rng.integers(0, n, size=nb)
    bl = rng.integers(1, 12, size=nb)
    rs, rd = [], []
    for u, s, l in zip(bu, bs, bl):
        for t in range(int(l)):
            if s + t < n:
                rs.append(u)
                rd.append(s + t)
    src = np.concatenate([src, np.array(rs, dtype=np.int64)])
    dst = np.concatenate([dst, np.array(rd, dtype=np.int64)])
    return csr_from_edges(n, src, dst, symmetric=symmetric)


def adjacency_lists(rowoff, cols):
    n = len(rowoff) - 1
    return [list(map(int, cols[int(rowoff[u]):int(rowoff[u + 1])])) for u in range(n)]
