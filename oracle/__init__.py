"""ctypes shim over oracle/liboracle.so — the plain CPU oracle (see gcgt_oracle.c for the paper citations).

TEST INFRASTRUCTURE ONLY: imported by tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
``--impl reference`` legs, never by the product package ``paper_conf_sigmod_shalt19_b200``.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "gcgt_oracle.c")
_SRC_PAR = os.path.join(_HERE, "gcgt_oracle_par.c")
_LIB = os.path.join(_HERE, "liboracle.so")

ERRORS = {0: "OK", -1: "EINVAL", -2: "EUNSORTED", -3: "ERANGE", -4: "ESEGLEN", -5: "ENOMEM", -8: "EFORMAT"}


class OracleError(RuntimeError):
    def __init__(self, code: int, what: str):
        super().__init__(f"oracle {what}: {ERRORS.get(code, code)}")
        self.code = code


def build(force: bool = False) -> str:
    """Compile the oracle (plain C, -O2; OpenMP only in gcgt_oracle_par.c).  Building the checker is not using it."""
    if (force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC)
            or os.path.getmtime(_LIB) < os.path.getmtime(_SRC_PAR)):
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-fPIC", "-shared", "-Wall", "-fopenmp", "-o", _LIB, _SRC,
                               _SRC_PAR])
    return _LIB


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = C.CDLL(_LIB)
        u64, i64, u32, i32, p = C.c_uint64, C.c_int64, C.c_uint32, C.c_int, C.c_void_p
        L.orc_vlc_len.restype = u64
        L.orc_vlc_len.argtypes = [i32, u64]
        L.orc_vlc_string.argtypes = [i32, u64, C.c_char_p, i32]
        L.orc_vlc_read.argtypes = [i32, p, u64, C.POINTER(u64), C.POINTER(u64)]
        L.orc_encode.argtypes = [u64, p, p, u32, u32, u32, C.POINTER(p), C.POINTER(u64), p]
        L.orc_encode_list.restype = i64
        L.orc_encode_list.argtypes = [u64, p, u64, u32, u32, u32, i32, C.c_char_p, u64]
        L.orc_free.argtypes = [p]
        L.orc_decode_vertex.argtypes = [p, u64, u64, u64, u32, u32, u32, p, u64, C.POINTER(u64), C.POINTER(u64)]
        L.orc_decode.argtypes = [u64, p, p, u32, u32, u32, p, p, u64]
        L.orc_alg4_trace.argtypes = [i32, p, u64, i32, i32, p, p, p, p, C.POINTER(i32)]
        L.orc_bfs.argtypes = [u64, p, p, u64, p]
        L.orc_bfs_cgr.argtypes = [u64, p, p, u32, u32, u32, u64, p, C.POINTER(u64)]
        L.orc_cc.argtypes = [u64, p, p, p]
        L.orc_bc.argtypes = [u64, p, p, p, u64, p]
        L.orc_bfs_cgr_par.argtypes = [u64, p, p, u32, u32, u32, u64, p, C.POINTER(u64), i32]
        L.orc_bfs_par.argtypes = [u64, p, p, u64, p, i32]
        L.orc_bfs_cgr_sample.argtypes = [u64, p, p, u32, u32, u32, u64, p, C.POINTER(u64), i32, u64]
        L.orc_max_threads.restype = i32
        L.orc_encode_par.argtypes = [u64, p, p, u32, u32, u32, C.POINTER(p), C.POINTER(u64), p, i32]
        L.orc_bc_par.argtypes = [u64, p, p, p, u64, p, i32]
        _lib = L
    return _lib


def _ptr(a: np.ndarray):
    return a.ctypes.data_as(C.c_void_p)


def _csr(rowoff, cols):
    rowoff = np.ascontiguousarray(rowoff, dtype=np.uint64)
    cols = np.ascontiguousarray(cols, dtype=np.uint32)
    if cols.size == 0:
        cols = np.zeros(1, dtype=np.uint32)
    return rowoff, cols


# ----------------------------------------------------------------------------------------------------------------
# VLC (App. B, Table 3)
# ----------------------------------------------------------------------------------------------------------------
def vlc_len(k: int, x: int) -> int:
    return int(lib().orc_vlc_len(k, x))


def vlc_string(k: int, x: int) -> str:
    buf = C.create_string_buffer(256)
    n = lib().orc_vlc_string(k, x, buf, 256)
    if n < 0:
        raise OracleError(n, "vlc_string")
    return buf.value.decode()


def bits_to_bytes(bits: str) -> tuple[np.ndarray, int]:
    """'0'/'1' string -> MSB-first bytes (FORMAT.md R1), plus the bit count."""
    nb = len(bits)
    out = np.zeros((nb + 7) // 8 + 16, dtype=np.uint8)
    for i, ch in enumerate(bits):
        if ch == "1":
            out[i >> 3] |= 0x80 >> (i & 7)
    return out, nb


def bytes_to_bits(b: np.ndarray, nbits: int) -> str:
    b = np.asarray(b, dtype=np.uint8)
    return "".join("1" if (b[i >> 3] >> (7 - (i & 7))) & 1 else "0" for i in range(nbits))


def vlc_read(k: int, bytes_: np.ndarray, nbits: int, pos: int) -> tuple[int, int]:
    p = C.c_uint64(pos)
    v = C.c_uint64(0)
    st = lib().orc_vlc_read(k, _ptr(bytes_), nbits, C.byref(p), C.byref(v))
    if st != 0:
        raise OracleError(-8, "vlc_read")
    return int(v.value), int(p.value)


# ----------------------------------------------------------------------------------------------------------------
# Encoder / decoder (§3.1, App. C, §5.2; FORMAT.md)
# ----------------------------------------------------------------------------------------------------------------
def encode_list(u, adj, min_interval_len=4, residual_segment_len=32, zeta_k=3, illustrative=False) -> str:
    """One vertex record as a '0'/'1' string (hand-worked pins; illustrative=True is Fig. 2's raw mode)."""
    a = np.ascontiguousarray(adj, dtype=np.uint32)
    if a.size == 0:
        a = np.zeros(1, dtype=np.uint32)
        deg = 0
    else:
        deg = a.size
    cap = 64 * (deg + 8) + 8 * residual_segment_len * (deg + 2) + 256
    buf = C.create_string_buffer(cap)
    n = lib().orc_encode_list(u, _ptr(a), deg, min_interval_len, residual_segment_len, zeta_k,
                              1 if illustrative else 0, buf, cap)
    if n < 0:
        raise OracleError(int(n), "encode_list")
    return buf.value.decode()


def encode(rowoff, cols, min_interval_len=4, residual_segment_len=32, zeta_k=3):
    """CSR -> (bytes u8[ceil(nbits/8)], nbits, bit_offsets u64[n+1])."""
    rowoff, cols = _csr(rowoff, cols)
    n = rowoff.size - 1
    offs = np.zeros(n + 1, dtype=np.uint64)
    bp = C.c_void_p()
    nb = C.c_uint64(0)
    st = lib().orc_encode(n, _ptr(rowoff), _ptr(cols), min_interval_len, residual_segment_len, zeta_k,
                          C.byref(bp), C.byref(nb), _ptr(offs))
    if st != 0:
        raise OracleError(st, "encode")
    nbytes = (nb.value + 7) // 8
    out = np.frombuffer(C.string_at(bp.value, max(nbytes, 1)), dtype=np.uint8)[:nbytes].copy()
    lib().orc_free(bp)
    return out, int(nb.value), offs


def encode_par(rowoff, cols, min_interval_len=4, residual_segment_len=32, zeta_k=3, threads: int = 0):
    """Same output as encode(), records encoded per vertex in parallel and concatenated (gcgt_oracle_par.c)."""
    rowoff, cols = _csr(rowoff, cols)
    n = rowoff.size - 1
    offs = np.zeros(n + 1, dtype=np.uint64)
    bp = C.c_void_p()
    nb = C.c_uint64(0)
    st = lib().orc_encode_par(n, _ptr(rowoff), _ptr(cols), min_interval_len, residual_segment_len, zeta_k,
                              C.byref(bp), C.byref(nb), _ptr(offs), threads)
    if st != 0:
        raise OracleError(st, "encode_par")
    nbytes = (nb.value + 7) // 8
    out = np.empty(max(nbytes, 1), dtype=np.uint8)
    C.memmove(out.ctypes.data, bp.value, max(nbytes, 1))
    lib().orc_free(bp)
    return out[:nbytes], int(nb.value), offs


def _padded(bytes_):
    b = np.zeros(np.asarray(bytes_).size + 16, dtype=np.uint8)
    b[: np.asarray(bytes_).size] = bytes_
    return b


def decode_vertex(bytes_, nbits, start, u, min_interval_len, residual_segment_len, zeta_k, cap=1 << 20):
    b = _padded(bytes_)
    out = np.zeros(cap, dtype=np.uint32)
    d = C.c_uint64(0)
    end = C.c_uint64(0)
    st = lib().orc_decode_vertex(_ptr(b), nbits, start, u, min_interval_len, residual_segment_len, zeta_k,
                                 _ptr(out), cap, C.byref(d), C.byref(end))
    if st != 0:
        raise OracleError(st, "decode_vertex")
    return out[: d.value].copy(), int(end.value)


def decode(bytes_, bit_offsets, min_interval_len, residual_segment_len, zeta_k, m_cap):
    b = _padded(bytes_)
    offs = np.ascontiguousarray(bit_offsets, dtype=np.uint64)
    n = offs.size - 1
    rowoff = np.zeros(n + 1, dtype=np.uint64)
    cols = np.zeros(max(m_cap, 1), dtype=np.uint32)
    st = lib().orc_decode(n, _ptr(b), _ptr(offs), min_interval_len, residual_segment_len, zeta_k,
                          _ptr(rowoff), _ptr(cols), m_cap)
    if st != 0:
        raise OracleError(st, "decode")
    return rowoff, cols[: int(rowoff[-1])].copy()


def alg4_trace(bits: str, K: int, zeta_k: int = 1, max_rounds: int = 16):
    """Alg. 4 / Fig. 5 emulation. Returns (vals[K], poss[rounds][K], flags[rounds][K], results, nrounds)."""
    b, nb = bits_to_bytes(bits)
    vals = np.zeros(K, dtype=np.uint64)
    tp = np.zeros(max_rounds * K, dtype=np.int64)
    tf = np.zeros(max_rounds * K, dtype=np.int32)
    res = np.zeros(K, dtype=np.uint64)
    tot = C.c_int(0)
    r = lib().orc_alg4_trace(zeta_k, _ptr(b), nb, K, max_rounds, _ptr(vals), _ptr(tp), _ptr(tf), _ptr(res),
                             C.byref(tot))
    if r < 0:
        raise OracleError(r, "alg4_trace")
    rr = min(r, max_rounds)
    return vals, tp[: rr * K].reshape(rr, K), tf[: rr * K].reshape(rr, K), res[: tot.value].copy(), r


# ----------------------------------------------------------------------------------------------------------------
# Applications (§6, Fig. 7)
# ----------------------------------------------------------------------------------------------------------------
def bfs(rowoff, cols, source: int) -> np.ndarray:
    rowoff, cols = _csr(rowoff, cols)
    n = rowoff.size - 1
    lv = np.zeros(n, dtype=np.int32)
    st = lib().orc_bfs(n, _ptr(rowoff), _ptr(cols), source, _ptr(lv))
    if st != 0:
        raise OracleError(st, "bfs")
    return lv


def bfs_cgr(bytes_, bit_offsets, min_interval_len, residual_segment_len, zeta_k, source: int):
    b = _padded(bytes_)
    offs = np.ascontiguousarray(bit_offsets, dtype=np.uint64)
    n = offs.size - 1
    lv = np.zeros(n, dtype=np.int32)
    e = C.c_uint64(0)
    st = lib().orc_bfs_cgr(n, _ptr(b), _ptr(offs), min_interval_len, residual_segment_len, zeta_k, source,
                           _ptr(lv), C.byref(e))
    if st != 0:
        raise OracleError(st, "bfs_cgr")
    return lv, int(e.value)


def bfs_par(rowoff, cols, source: int, threads: int = 0) -> np.ndarray:
    """Level-synchronous OpenMP BFS over the CSR (gcgt_oracle_par.c); threads = 0: all cores."""
    rowoff, cols = _csr(rowoff, cols)
    n = rowoff.size - 1
    lv = np.zeros(n, dtype=np.int32)
    st = lib().orc_bfs_par(n, _ptr(rowoff), _ptr(cols), source, _ptr(lv), threads)
    if st != 0:
        raise OracleError(st, "bfs_par")
    return lv


def bfs_cgr_par(bytes_, bit_offsets, min_interval_len, residual_segment_len, zeta_k, source: int, threads: int = 0):
    """Level-synchronous OpenMP BFS decoding the oracle's own CGR; returns (levels, edges)."""
    b = _padded(bytes_)
    offs = np.ascontiguousarray(bit_offsets, dtype=np.uint64)
    n = offs.size - 1
    lv = np.zeros(n, dtype=np.int32)
    e = C.c_uint64(0)
    st = lib().orc_bfs_cgr_par(n, _ptr(b), _ptr(offs), min_interval_len, residual_segment_len, zeta_k, source,
                               _ptr(lv), C.byref(e), threads)
    if st != 0:
        raise OracleError(st, "bfs_cgr_par")
    return lv, int(e.value)


def bc_par(rowoff, cols, sources, threads: int = 0) -> np.ndarray:
    """Brandes BC parallel over sources, summed in source order (bit-identical to bc())."""
    rowoff, cols = _csr(rowoff, cols)
    n = rowoff.size - 1
    src = np.ascontiguousarray(sources, dtype=np.uint32)
    out = np.zeros(n, dtype=np.float64)
    st = lib().orc_bc_par(n, _ptr(rowoff), _ptr(cols), _ptr(src) if src.size else None, src.size, _ptr(out), threads)
    if st != 0:
        raise OracleError(st, "bc_par")
    return out


def bfs_cgr_sample(bytes_, bit_offsets, min_interval_len, residual_segment_len, zeta_k, source: int,
                   max_edges: int, threads: int = 0) -> int:
    """Timing sample: the BFS's first whole levels until >= max_edges arcs are decoded; returns the arcs decoded."""
    b = _padded(bytes_)
    offs = np.ascontiguousarray(bit_offsets, dtype=np.uint64)
    n = offs.size - 1
    lv = np.zeros(n, dtype=np.int32)
    e = C.c_uint64(0)
    st = lib().orc_bfs_cgr_sample(n, _ptr(b), _ptr(offs), min_interval_len, residual_segment_len, zeta_k, source,
                                  _ptr(lv), C.byref(e), threads, max_edges)
    if st != 0:
        raise OracleError(st, "bfs_cgr_sample")
    return int(e.value)


def max_threads() -> int:
    return int(lib().orc_max_threads())


def cc(rowoff, cols) -> np.ndarray:
    rowoff, cols = _csr(rowoff, cols)
    n = rowoff.size - 1
    lab = np.zeros(n, dtype=np.uint32)
    st = lib().orc_cc(n, _ptr(rowoff), _ptr(cols), _ptr(lab))
    if st != 0:
        raise OracleError(st, "cc")
    return lab


def bc(rowoff, cols, sources) -> np.ndarray:
    rowoff, cols = _csr(rowoff, cols)
    n = rowoff.size - 1
    src = np.ascontiguousarray(sources, dtype=np.uint32)
    out = np.zeros(n, dtype=np.float64)
    st = lib().orc_bc(n, _ptr(rowoff), _ptr(cols), _ptr(src) if src.size else None, src.size, _ptr(out))
    if st != 0:
        raise OracleError(st, "bc")
    return out
