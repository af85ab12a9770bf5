"""Seeded synthetic inputs (shared by the oracle side and the product side; holds none of the method's arithmetic).

Graph recipes are DESIGN.md §4 / SURVEY.md §8(d); the C++ generators live in synth.cpp.  ``CONFIGS`` names the
BASELINE.json configurations (c1..c5) plus scaled-down variants used by the parity tests.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess
from dataclasses import dataclass

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "synth.cpp")
_LIB = os.path.join(_HERE, "libsynth.so")


def build(force: bool = False) -> str:
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        subprocess.check_call(["g++", "-O3", "-std=c++17", "-fopenmp", "-fPIC", "-shared", "-o", _LIB, _SRC])
    return _LIB


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = C.CDLL(_LIB)
        p, u64, i32, d = C.c_void_p, C.c_uint64, C.c_int, C.c_double
        L.syn_n.restype = u64
        L.syn_n.argtypes = [p]
        L.syn_m.restype = u64
        L.syn_m.argtypes = [p]
        L.syn_copy.argtypes = [p, p, p]
        L.syn_free.argtypes = [p]
        L.syn_rmat.restype = p
        L.syn_rmat.argtypes = [i32, i32, u64, d, d, d]
        L.syn_web.restype = p
        L.syn_web.argtypes = [u64, d, u64, i32]
        L.syn_social.restype = p
        L.syn_social.argtypes = [u64, d, u64, u64, i32]
        L.syn_rmat_slice.restype = p
        L.syn_rmat_slice.argtypes = [i32, i32, u64, d, d, d, u64, u64]
        L.syn_rmat_counts.argtypes = [i32, i32, u64, d, d, d, p]
        _lib = L
    return _lib


def _take(h):
    if not h:
        raise MemoryError("synthetic generator failed (out of memory?)")
    L = lib()
    n, m = int(L.syn_n(h)), int(L.syn_m(h))
    rowoff = np.empty(n + 1, dtype=np.uint64)
    cols = np.empty(max(m, 1), dtype=np.uint32)
    L.syn_copy(h, rowoff.ctypes.data_as(C.c_void_p), cols.ctypes.data_as(C.c_void_p))
    L.syn_free(h)
    return rowoff, cols[:m]


def rmat(scale: int, edgefactor: int = 16, seed: int = 1, A=0.57, B=0.19, Cc=0.19):
    return _take(lib().syn_rmat(scale, edgefactor, seed, A, B, Cc))


def rmat_slice(scale: int, edgefactor: int, seed: int, lo: int, hi: int, A=0.57, B=0.19, Cc=0.19):
    """Rows [lo, hi) of rmat(scale, edgefactor, seed) (global column ids), generated without the rest of the graph."""
    return _take(lib().syn_rmat_slice(scale, edgefactor, seed, A, B, Cc, lo, hi))


def rmat_slices(scale: int, edgefactor: int, seed: int, parts: int, A=0.57, B=0.19, Cc=0.19):
    """Vertex-range boundaries (multiples of 32) splitting rmat(...) into `parts` slices of about equal arc counts
    (from the pre-deduplication counts)."""
    n = 1 << scale
    counts = np.empty(n, dtype=np.uint32)
    lib().syn_rmat_counts(scale, edgefactor, seed, A, B, Cc, counts.ctypes.data_as(C.c_void_p))
    pre = np.concatenate([[0], np.cumsum(counts.astype(np.uint64))])
    tot = int(pre[-1])
    b = [0]
    for r in range(1, parts):
        v = int(np.searchsorted(pre, tot * r // parts)) // 32 * 32
        b.append(max(b[-1], min(n, v)))
    b.append(n)
    return b


def web(n: int, mean_deg: float = 16.1, seed: int = 2002, relabel: bool = True):
    return _take(lib().syn_web(n, mean_deg, seed, 1 if relabel else 0))


def social(n: int, mean_deg: float = 35.3, max_deg: int = 3_000_000, seed: int = 2010, relabel: bool = True):
    return _take(lib().syn_social(n, mean_deg, max_deg, seed, 1 if relabel else 0))


@dataclass(frozen=True)
class Config:
    name: str
    kind: str           # rmat | web | social
    args: tuple
    symmetric: bool     # TEPS halves the arc count on symmetrised R-MAT (Graph500 convention)
    min_interval_len: int = 4
    residual_segment_len: int = 32
    zeta_k: int = 3
    desc: str = ""

    def make(self):
        if self.kind == "rmat":
            return rmat(*self.args)
        if self.kind == "web":
            return web(*self.args)
        if self.kind == "social":
            return social(*self.args)
        raise ValueError(self.kind)


CONFIGS = {
    # BASELINE.json configs[0]: R-MAT s10 ef16, minLen 4, residual segment 64 (bytes, FORMAT.md R15), BFS from 0
    "c1": Config("c1", "rmat", (10, 16, 1), True, 4, 64, 3, "R-MAT s10 ef16 seed 1 (symmetrised)"),
    # configs[1]: uk-2002-like web graph, BFS-reordered (Table 1 :1420: 18.5M / 298M)
    "c2": Config("c2", "web", (18_520_486, 15.3, 2002), False, 4, 32, 3, "uk-2002-like web, 18.5M vertices"),
    # configs[2]: twitter-like social graph (Table 1 :1423: 41.6M / 1.46B)
    "c3": Config("c3", "social", (41_652_230, 35.3, 3_000_000, 2010), False, 4, 32, 3,
                 "twitter-like social, 41.7M vertices"),
    # configs[3]: uk-2007-like web graph (Table 1 :1421: 105,896,555 vertices / 3,738,733,648 arcs).  The recipe's
    # mean-degree knob is the pre-deduplication target: 45.9 gives 35.3 distinct arcs per vertex (calibrated on a
    # 10M-vertex sample of the recipe: 44.0 -> 34.23, 46.0 -> 35.38), i.e. m ~ 3.74B
    "c4": Config("c4", "web", (105_896_555, 45.9, 2007), False, 4, 32, 3, "uk-2007-like web, 105.9M vertices"),
    # configs[4]: R-MAT s29 ef16
    "c5": Config("c5", "rmat", (29, 16, 29), True, 4, 32, 3, "R-MAT s29 ef16 seed 29 (symmetrised)"),
    # scaled-down variants of the same recipes for parity tests (oracle finishes in seconds)
    "web_s": Config("web_s", "web", (200_000, 16.1, 2002), False, 4, 32, 3, "web recipe, 200K vertices"),
    "social_s": Config("social_s", "social", (100_000, 35.3, 20_000, 2010), False, 4, 32, 3,
                       "social recipe, 100K vertices"),
    "rmat_s": Config("rmat_s", "rmat", (16, 16, 16), True, 4, 32, 3, "R-MAT s16 ef16"),
    # mid-size variants for performance sweeps
    "rmat_m": Config("rmat_m", "rmat", (22, 16, 22), True, 4, 32, 3, "R-MAT s22 ef16"),
    "social_m": Config("social_m", "social", (4_000_000, 35.3, 300_000, 2010), False, 4, 32, 3,
                       "social recipe, 4M vertices"),
}


def pick_roots(rowoff, count: int, seed: int = 20190630, exclude_dead: bool = True):
    """Seeded roots, uniform among vertices with out-degree > 0 (BASELINE.md seeds)."""
    deg = np.diff(rowoff.astype(np.int64))
    cand = np.flatnonzero(deg > 0) if exclude_dead else np.arange(deg.size)
    rng = np.random.default_rng(seed)
    return [int(x) for x in rng.choice(cand, size=count, replace=True)] if cand.size else [0] * count


def bc_sources(rowoff, count: int = 64, seed: int = 64):
    return pick_roots(rowoff, count, seed)
