"""paper_conf_sigmod_shalt19_b200 — thin Python binding over libgcgt.so (include/gcgt.h).

Argument marshalling only: every step of the hot path runs in the library (host C++ encoder + sm_100a kernels).
There is no CPU fallback: if libgcgt.so is missing or no CUDA device is usable, calls raise ``GcgtError``.
PyTorch is used (optionally) for device memory and streams: output tensors on ``cuda`` are written in place via
``GCGT_OUT_DEVICE``; the graph runs on the caller's current torch stream when ``stream="torch"``.
"""
from __future__ import annotations

import ctypes as C
import os

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("GCGT_LIB") or os.path.join(_HERE, "libgcgt.so")  # GCGT_LIB: A/B builds (tools/)

OK, EINVAL, EUNSORTED, ERANGE, ESEGLEN, ENOMEM, ECUDA, EFORMAT = 0, -1, -2, -3, -4, -5, -6, -8
STATUS_NAMES = {0: "OK", -1: "EINVAL", -2: "EUNSORTED", -3: "ERANGE", -4: "ESEGLEN", -5: "ENOMEM", -6: "ECUDA",
                -8: "EFORMAT"}
OUT_HOST, OUT_DEVICE = 0, 1

# public symbols of include/gcgt.h (tests check the library exports every one)
ABI_SYMBOLS = ["gcgt_encode", "gcgt_encode_transpose", "gcgt_encode_slice", "gcgt_cgr_concat", "gcgt_cgr_slice_info", "gcgt_cgr_view", "gcgt_cgr_from_arrays", "gcgt_cgr_save", "gcgt_cgr_open",
               "gcgt_cgr_pin",
               "gcgt_cgr_free", "gcgt_load", "gcgt_load_csr", "gcgt_unload", "gcgt_profile", "gcgt_profile_spans", "gcgt_graph_range", "gcgt_bfs", "gcgt_cc", "gcgt_bc",
               "gcgt_dist_bfs_begin", "gcgt_dist_bfs_expand", "gcgt_dist_bfs_commit", "gcgt_dist_bfs_absorb",
               "gcgt_dist_bfs_levels", "gcgt_dist_cc_hook", "gcgt_dist_cc_merge", "gcgt_dist_cc_jump", "gcgt_sync",
               "gcgt_debug_warp_decode", "gcgt_last_error", "gcgt_version"]


class GcgtError(RuntimeError):
    def __init__(self, status: int, what: str, msg: str = ""):
        super().__init__(f"{what}: {STATUS_NAMES.get(status, status)} {msg}".strip())
        self.status = status


class Params(C.Structure):
    _fields_ = [("min_interval_len", C.c_uint32), ("residual_segment_len", C.c_uint32), ("zeta_k", C.c_uint32)]


class Csr(C.Structure):
    _fields_ = [("n", C.c_uint64), ("row_offsets", C.c_void_p), ("cols", C.c_void_p)]


class Stats(C.Structure):
    _fields_ = [("iterations", C.c_uint32), ("reserved", C.c_uint32), ("vertices_expanded", C.c_uint64),
                ("arcs_decoded", C.c_uint64), ("cgr_bits_decoded", C.c_uint64), ("device_ms", C.c_double),
                ("kernel_ms", C.c_double), ("kernel_launches", C.c_uint64), ("launches", C.c_uint64)]

    def as_dict(self):
        return {k: getattr(self, k) for k, _ in self._fields_ if k != "reserved"}


class LoadOpts(C.Structure):
    _fields_ = [("device", C.c_int), ("stream", C.c_void_p), ("rank", C.c_int), ("nranks", C.c_int),
                ("reserved", C.c_void_p), ("in_cgr", C.c_void_p), ("symmetric", C.c_int),
                ("direction_optimizing", C.c_int), ("host_resident", C.c_int)]


_lib = None


def lib():
    """Loads libgcgt.so (built by build.py / __graft_entry__.build()).  Fails loudly if it is missing."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise GcgtError(ECUDA, "libgcgt.so not built", f"({LIB_PATH}); run __graft_entry__.build()")
        L = C.CDLL(LIB_PATH)
        p, u32, u64, i32 = C.c_void_p, C.c_uint32, C.c_uint64, C.c_int
        L.gcgt_encode.argtypes = [C.POINTER(Csr), C.POINTER(Params), C.POINTER(p)]
        L.gcgt_encode_transpose.argtypes = [C.POINTER(Csr), C.POINTER(Params), C.POINTER(p)]
        L.gcgt_encode_slice.argtypes = [C.POINTER(Csr), u64, u64, C.POINTER(Params), C.POINTER(p)]
        L.gcgt_cgr_concat.argtypes = [C.POINTER(p), u32, C.POINTER(p)]
        L.gcgt_cgr_slice_info.argtypes = [p, C.POINTER(u64), C.POINTER(u64)]
        L.gcgt_cgr_view.argtypes = [p, C.POINTER(p), C.POINTER(u64), C.POINTER(p), C.POINTER(u64), C.POINTER(Params)]
        L.gcgt_cgr_from_arrays.argtypes = [u64, p, u64, p, C.POINTER(Params), C.POINTER(p)]
        L.gcgt_cgr_save.argtypes = [p, C.c_char_p]
        L.gcgt_cgr_pin.argtypes = [p]
        L.gcgt_cgr_open.argtypes = [C.c_char_p, C.POINTER(p)]
        L.gcgt_cgr_free.argtypes = [p]
        L.gcgt_cgr_free.restype = None
        L.gcgt_load.argtypes = [p, C.POINTER(LoadOpts), C.POINTER(p)]
        L.gcgt_load_csr.argtypes = [C.POINTER(Csr), C.POINTER(LoadOpts), C.POINTER(p)]
        L.gcgt_unload.argtypes = [p]
        L.gcgt_unload.restype = None
        L.gcgt_profile.argtypes = [p, i32]
        L.gcgt_profile_spans.argtypes = [p, p, i32]
        L.gcgt_graph_range.argtypes = [p, C.POINTER(u64), C.POINTER(u64)]
        L.gcgt_bfs.argtypes = [p, u32, p, i32, C.POINTER(Stats)]
        L.gcgt_cc.argtypes = [p, p, i32, C.POINTER(Stats)]
        L.gcgt_bc.argtypes = [p, p, u32, p, i32, C.POINTER(Stats)]
        L.gcgt_dist_bfs_begin.argtypes = [p, u32]
        L.gcgt_dist_bfs_expand.argtypes = [p, u32, p, p, i32]
        L.gcgt_dist_bfs_commit.argtypes = [p, u32, p, u32, p, i32]
        L.gcgt_dist_bfs_absorb.argtypes = [p, p, C.POINTER(u64)]
        L.gcgt_dist_bfs_levels.argtypes = [p, p, i32]
        L.gcgt_dist_cc_hook.argtypes = [p, p, p, u64, C.POINTER(u64)]
        L.gcgt_dist_cc_merge.argtypes = [p, p, p, u64]
        L.gcgt_dist_cc_jump.argtypes = [p, p]
        L.gcgt_sync.argtypes = [p]
        L.gcgt_debug_warp_decode.argtypes = [p, u64, u32, u32, u64, p, p, p, C.POINTER(u32)]
        L.gcgt_last_error.restype = C.c_char_p
        L.gcgt_version.restype = C.c_char_p
        _lib = L
    return _lib


def _check(st: int, what: str):
    if st != OK:
        raise GcgtError(st, what, lib().gcgt_last_error().decode(errors="replace"))


def _np_ptr(a: np.ndarray):
    return C.c_void_p(a.ctypes.data)


class CGR:
    """Host CGR (library-owned).  Build with ``encode`` / ``from_arrays`` / ``open``."""

    def __init__(self, handle: C.c_void_p):
        self._h = handle

    @property
    def handle(self):
        return self._h

    def view(self):
        """(bytes u8[ceil(nbits/8)], nbits, bit_offsets u64[n+1], n, (min_interval_len, residual_segment_len, zeta_k));
        numpy arrays are copies."""
        b, off = C.c_void_p(), C.c_void_p()
        nbits, n = C.c_uint64(), C.c_uint64()
        P = Params()
        _check(lib().gcgt_cgr_view(self._h, C.byref(b), C.byref(nbits), C.byref(off), C.byref(n), C.byref(P)),
               "gcgt_cgr_view")
        nbytes = (nbits.value + 7) // 8
        by = np.ctypeslib.as_array((C.c_uint8 * max(nbytes, 1)).from_address(b.value))[:nbytes].copy()
        bo = np.ctypeslib.as_array((C.c_uint64 * (n.value + 1)).from_address(off.value)).copy()
        return by, int(nbits.value), bo, int(n.value), (P.min_interval_len, P.residual_segment_len, P.zeta_k)

    def pin(self):
        """gcgt_cgr_pin: build the derived load tables now and page-lock the host arrays (fast repeated loads)."""
        _check(lib().gcgt_cgr_pin(self._h), "gcgt_cgr_pin")
        return self

    def save(self, path: str):
        _check(lib().gcgt_cgr_save(self._h, path.encode()), "gcgt_cgr_save")

    def free(self):
        if self._h:
            lib().gcgt_cgr_free(self._h)
            self._h = None

    def __del__(self):
        try:
            self.free()
        except Exception:
            pass


def encode(row_offsets: np.ndarray, cols: np.ndarray, min_interval_len: int = 4, residual_segment_len: int = 32,
           zeta_k: int = 3) -> CGR:
    ro = np.ascontiguousarray(row_offsets, dtype=np.uint64)
    co = np.ascontiguousarray(cols, dtype=np.uint32)
    if co.size == 0:
        co = np.zeros(1, dtype=np.uint32)
    csr = Csr(ro.size - 1, ro.ctypes.data, co.ctypes.data)
    P = Params(min_interval_len, residual_segment_len, zeta_k)
    h = C.c_void_p()
    _check(lib().gcgt_encode(C.byref(csr), C.byref(P), C.byref(h)), "gcgt_encode")
    return CGR(h)


def encode_transpose(row_offsets: np.ndarray, cols: np.ndarray, min_interval_len: int = 4,
                     residual_segment_len: int = 32, zeta_k: int = 3) -> CGR:
    """CGR of the transpose (in-arcs), for Graph(..., in_cgr=...) bottom-up steps."""
    ro = np.ascontiguousarray(row_offsets, dtype=np.uint64)
    co = np.ascontiguousarray(cols, dtype=np.uint32)
    if co.size == 0:
        co = np.zeros(1, dtype=np.uint32)
    csr = Csr(ro.size - 1, ro.ctypes.data, co.ctypes.data)
    P = Params(min_interval_len, residual_segment_len, zeta_k)
    h = C.c_void_p()
    _check(lib().gcgt_encode_transpose(C.byref(csr), C.byref(P), C.byref(h)), "gcgt_encode_transpose")
    return CGR(h)


def encode_slice(row_offsets: np.ndarray, cols: np.ndarray, first: int, n_total: int, min_interval_len: int = 4,
                 residual_segment_len: int = 32, zeta_k: int = 3) -> CGR:
    """Records of vertices first .. first + len(row_offsets) - 2 (rows of a slice CSR, global column ids)."""
    ro = np.ascontiguousarray(row_offsets, dtype=np.uint64)
    co = np.ascontiguousarray(cols, dtype=np.uint32)
    if co.size == 0:
        co = np.zeros(1, dtype=np.uint32)
    csr = Csr(ro.size - 1, ro.ctypes.data, co.ctypes.data)
    P = Params(min_interval_len, residual_segment_len, zeta_k)
    h = C.c_void_p()
    _check(lib().gcgt_encode_slice(C.byref(csr), first, n_total, C.byref(P), C.byref(h)), "gcgt_encode_slice")
    return CGR(h)


def concat(parts) -> CGR:
    """One CGR from consecutive slices (gcgt_cgr_concat)."""
    arr = (C.c_void_p * len(parts))(*[p.handle for p in parts])
    h = C.c_void_p()
    _check(lib().gcgt_cgr_concat(arr, len(parts), C.byref(h)), "gcgt_cgr_concat")
    return CGR(h)


def slice_info(cgr: CGR):
    """(first vertex, n_total) of a CGR (0, n for a whole graph)."""
    b, t = C.c_uint64(), C.c_uint64()
    _check(lib().gcgt_cgr_slice_info(cgr.handle, C.byref(b), C.byref(t)), "gcgt_cgr_slice_info")
    return int(b.value), int(t.value)


def from_arrays(bytes_: np.ndarray, nbits: int, bit_offsets: np.ndarray, min_interval_len: int,
                residual_segment_len: int, zeta_k: int) -> CGR:
    b = np.ascontiguousarray(bytes_, dtype=np.uint8)
    if b.size == 0:
        b = np.zeros(1, dtype=np.uint8)
    bo = np.ascontiguousarray(bit_offsets, dtype=np.uint64)
    P = Params(min_interval_len, residual_segment_len, zeta_k)
    h = C.c_void_p()
    _check(lib().gcgt_cgr_from_arrays(bo.size - 1, _np_ptr(b), nbits, _np_ptr(bo), C.byref(P), C.byref(h)),
           "gcgt_cgr_from_arrays")
    return CGR(h)


def open_cgr(path: str) -> CGR:
    h = C.c_void_p()
    _check(lib().gcgt_cgr_open(path.encode(), C.byref(h)), "gcgt_cgr_open")
    return CGR(h)


CUDA_STREAM_LEGACY = 1  # cudaStreamLegacy: the legacy default stream, torch's default stream


def _torch_stream(device):
    """Torch's current stream on `device` as a cudaStream_t value: the legacy default stream is handle 0 in torch, which
    the C ABI reads as "no stream" (a library-created one), so it is passed as cudaStreamLegacy."""
    import torch
    s = torch.cuda.current_stream(device).cuda_stream
    return s if s else CUDA_STREAM_LEGACY


def _out(out, n, np_dtype, torch_dtype_name):
    """Returns (pointer, placement, result_object)."""
    if out is None:
        a = np.empty(n, dtype=np_dtype)
        return _np_ptr(a), OUT_HOST, a
    if isinstance(out, np.ndarray):
        if out.dtype != np_dtype or out.size != n or not out.flags.c_contiguous:
            raise GcgtError(EINVAL, "output array", f"need contiguous {np_dtype} of size {n}")
        return _np_ptr(out), OUT_HOST, out
    # torch tensor
    import torch
    if out.dtype != getattr(torch, torch_dtype_name) or out.numel() != n or not out.is_contiguous():
        raise GcgtError(EINVAL, "output tensor", f"need contiguous {torch_dtype_name} of size {n}")
    return C.c_void_p(out.data_ptr()), (OUT_DEVICE if out.is_cuda else OUT_HOST), out


class Graph:
    """Device-resident CGR (gcgt_load)."""

    def __init__(self, cgr: CGR, device: int = 0, stream=None, rank: int = 0, nranks: int = 1,
                 in_cgr: "CGR | None" = None, symmetric: bool = False, direction_optimizing: bool = True,
                 host_resident: bool = False):
        self.stream_kind = stream if isinstance(stream, str) else ("caller" if stream else "own")
        if stream == "torch":
            stream = _torch_stream(device)
        opts = LoadOpts(device, C.c_void_p(stream) if stream else None, rank, nranks, None,
                        in_cgr.handle if in_cgr is not None else None,
                        1 if symmetric else 0, 1 if direction_optimizing else 0, 1 if host_resident else 0)
        self._in_cgr = in_cgr
        self.has_in = in_cgr is not None or bool(symmetric)
        h = C.c_void_p()
        _check(lib().gcgt_load(cgr.handle, C.byref(opts), C.byref(h)), "gcgt_load")
        self._h = h
        self.n = slice_info(cgr)[1]
        self.last_stats: dict = {}

    def profile(self, enable: bool = True, spans: bool = False):
        """Kernel timing (gcgt_stats.kernel_ms); spans=True also per-level spans (the level loop then waits per
        level)."""
        _check(lib().gcgt_profile(self._h, (2 if spans else 1) if enable else 0), "gcgt_profile")

    def profile_spans(self):
        """Last profiled gcgt_bfs split into spans (ms): expand, hub, bottom-up, contraction."""
        a = np.zeros(4, dtype=np.float64)
        _check(lib().gcgt_profile_spans(self._h, _np_ptr(a), 4), "gcgt_profile_spans")
        return dict(zip(["expand", "hub", "bottom_up", "contract"], [float(x) for x in a]))

    def range(self):
        lo, hi = C.c_uint64(), C.c_uint64()
        _check(lib().gcgt_graph_range(self._h, C.byref(lo), C.byref(hi)), "gcgt_graph_range")
        return int(lo.value), int(hi.value)

    def bfs(self, source: int, out=None):
        ptr, where, res = _out(out, self.n, np.int32, "int32")
        st = Stats()
        _check(lib().gcgt_bfs(self._h, source, ptr, where, C.byref(st)), "gcgt_bfs")
        self.last_stats = st.as_dict()
        return res

    def cc(self, out=None):
        ptr, where, res = _out(out, self.n, np.uint32, "int32")
        st = Stats()
        _check(lib().gcgt_cc(self._h, ptr, where, C.byref(st)), "gcgt_cc")
        self.last_stats = st.as_dict()
        return res

    def bc(self, sources, out=None):
        src = np.ascontiguousarray(sources, dtype=np.uint32)
        ptr, where, res = _out(out, self.n, np.float64, "float64")
        st = Stats()
        _check(lib().gcgt_bc(self._h, _np_ptr(src) if src.size else None, src.size, ptr, where, C.byref(st)),
               "gcgt_bc")
        self.last_stats = st.as_dict()
        return res

    # ---- partitioned steps (dist.py); device pointers as ints; enqueued on the graph's stream ----------------------
    def dist_bfs_begin(self, source: int):
        _check(lib().gcgt_dist_bfs_begin(self._h, source), "gcgt_dist_bfs_begin")

    def dist_bfs_expand(self, level: int, cand_ptr: int, fslice_ptr: int = 0, bottom_up: bool = False):
        _check(lib().gcgt_dist_bfs_expand(self._h, level, C.c_void_p(cand_ptr), C.c_void_p(fslice_ptr) if fslice_ptr
                                          else None, 1 if bottom_up else 0), "gcgt_dist_bfs_expand")

    def dist_bfs_commit(self, level: int, recv_ptr: int, nparts: int, fslice_ptr: int, keep: bool = False):
        _check(lib().gcgt_dist_bfs_commit(self._h, level, C.c_void_p(recv_ptr) if recv_ptr else None, nparts,
                                          C.c_void_p(fslice_ptr), 1 if keep else 0), "gcgt_dist_bfs_commit")

    def dist_bfs_absorb(self, frontier_ptr: int) -> int:
        cnt = C.c_uint64(0)
        _check(lib().gcgt_dist_bfs_absorb(self._h, C.c_void_p(frontier_ptr), C.byref(cnt)), "gcgt_dist_bfs_absorb")
        return int(cnt.value)

    def sync(self):
        _check(lib().gcgt_sync(self._h), "gcgt_sync")

    def dist_bfs_levels(self, out):
        ptr, where, res = _out(out, self.range()[1] - self.range()[0], np.int32, "int32")
        _check(lib().gcgt_dist_bfs_levels(self._h, ptr, where), "gcgt_dist_bfs_levels")
        return res

    def dist_cc_hook(self, parent_ptr: int, pairs_ptr: int = 0, cap: int = 0) -> int:
        h = C.c_uint64(0)
        _check(lib().gcgt_dist_cc_hook(self._h, C.c_void_p(parent_ptr), C.c_void_p(pairs_ptr) if pairs_ptr else None,
                                       cap, C.byref(h)), "gcgt_dist_cc_hook")
        return int(h.value)

    def dist_cc_merge(self, parent_ptr: int, pairs_ptr: int, npairs: int):
        _check(lib().gcgt_dist_cc_merge(self._h, C.c_void_p(parent_ptr), C.c_void_p(pairs_ptr), npairs),
               "gcgt_dist_cc_merge")

    def dist_cc_jump(self, parent_ptr: int):
        _check(lib().gcgt_dist_cc_jump(self._h, C.c_void_p(parent_ptr)), "gcgt_dist_cc_jump")

    def unload(self):
        if self._h:
            lib().gcgt_unload(self._h)
            self._h = None

    def __del__(self):
        try:
            self.unload()
        except Exception:
            pass


def cgr_n(cgr: CGR) -> int:
    n = C.c_uint64()
    _check(lib().gcgt_cgr_view(cgr.handle, None, None, None, C.byref(n), None), "gcgt_cgr_view")
    return int(n.value)


def load(cgr: CGR, device: int = 0, stream=None, **kw) -> Graph:
    return Graph(cgr, device, stream, **kw)


def load_csr(row_offsets: np.ndarray, cols: np.ndarray, device: int = 0, stream=None, symmetric: bool = False,
             direction_optimizing: bool = True) -> Graph:
    """Uncompressed baseline (gcgt_load_csr, §8 f3): the same BFS machinery reading col[] instead of the CGR.
    Only ``bfs`` is supported on the returned graph."""
    ro = np.ascontiguousarray(row_offsets, dtype=np.uint64)
    co = np.ascontiguousarray(cols, dtype=np.uint32)
    if co.size == 0:
        co = np.zeros(1, dtype=np.uint32)
    if stream == "torch":
        stream = _torch_stream(device)
    csr = Csr(ro.size - 1, ro.ctypes.data, co.ctypes.data)
    opts = LoadOpts(device, C.c_void_p(stream) if stream else None, 0, 1, None, None, 1 if symmetric else 0,
                    1 if direction_optimizing else 0, 0)
    h = C.c_void_p()
    _check(lib().gcgt_load_csr(C.byref(csr), C.byref(opts), C.byref(h)), "gcgt_load_csr")
    g = Graph.__new__(Graph)
    g._in_cgr = None
    g.has_in = bool(direction_optimizing)
    g.stream_kind = "torch" if stream else "own"
    g._h = h
    g.n = int(ro.size - 1)
    g.last_stats = {}
    return g


def debug_warp_decode(bytes_: np.ndarray, nbits: int, zeta_k: int, window: int, count: int):
    """Test hook: (vals[count], trace_pos[rounds][window], trace_flags[rounds][window], rounds) from the device
    warp decoder (gcgt_debug_warp_decode)."""
    b = np.zeros(np.asarray(bytes_).size + 16, dtype=np.uint8)
    b[: np.asarray(bytes_).size] = bytes_
    vals = np.zeros(max(count, 1), dtype=np.uint64)
    tp = np.zeros(6 * 32, dtype=np.uint32)
    tf = np.zeros(6 * 32, dtype=np.uint32)
    r = C.c_uint32(0)
    _check(lib().gcgt_debug_warp_decode(_np_ptr(b), nbits, zeta_k, window, count, _np_ptr(vals), _np_ptr(tp),
                                        _np_ptr(tf), C.byref(r)), "gcgt_debug_warp_decode")
    n = r.value
    return (vals[:count], tp.reshape(6, 32)[:n, :window].astype(np.int64), tf.reshape(6, 32)[:n, :window],
            n)


def version() -> str:
    return lib().gcgt_version().decode()
