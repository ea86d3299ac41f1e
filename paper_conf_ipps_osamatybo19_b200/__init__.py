"""B200-native independent-set graph colouring (Osama et al., IPDPS-W 2019).

Thin ctypes binding over libgc.so, the C ABI declared in include/gc.h.  This
module only marshals arguments (torch tensors / numpy arrays -> pointers and
sizes); every step of the colouring runs in the CUDA kernels of csrc/.  There
is no CPU fallback: if libgc.so is missing or no sm_100 device is present the
calls raise.  PyTorch is used for device memory, streams and process groups.

    import paper_conf_ipps_osamatybo19_b200 as gcb
    g = gcb.Graph(n, row_offsets, col_indices)        # host or cuda tensors
    colors, n_colors = g.color(seed=1, variant=gcb.MAXMIN)
"""
from __future__ import annotations

import ctypes
import os
from dataclasses import dataclass

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("GC_LIB_PATH") or os.path.join(_HERE, "libgc.so")  # override: experiments

# include/gc.h constants
GC_OK = 0
STATUS = {-1: "GC_ERR_INVALID_ARG", -2: "GC_ERR_SELF_LOOP", -3: "GC_ERR_NOT_SYMMETRIC",
          -4: "GC_ERR_TOO_LARGE", -5: "GC_ERR_CUDA", -6: "GC_ERR_NCCL", -7: "GC_ERR_OOM"}
MAXMIN = 0
LUBY_MIS = 1
IS_ALG2 = 3      # Alg.2 as written (max-only IS)
JP_ALG4 = 4      # Alg.2 + Alg.4 (GraphBLAS Jones-Plassmann)


def MULTIHASH(h: int) -> int:
    return 2 | (h << 8)


HASH_TABLE_MAX = 64


def LDF(variant: int) -> int:
    """Largest-degree-first priorities (reading R21) for GC_MAXMIN,
    GC_LUBY_MIS, GC_IS_ALG2 and GC_JP_ALG4."""
    return variant | (1 << 16)


def HASH_IS(t: int) -> int:
    """The paper's Hash IS (Alg.6, deterministic readings R16-R20), table of t colours."""
    return 5 | (t << 8)


BORROW_DEVICE = 1 << 0
VALIDATE = 1 << 1
COMPACT = 1 << 2
OUT_LOCAL_SLICE = 1 << 3
PROFILE = 1 << 4
MODE_AUTO, MODE_SWEEP, MODE_EVENT, MODE_EVENT_MULTI, MODE_COUNT = 0, 1, 2, 3, 4

EXPORTS = ["gc_create_csr", "gc_color", "gc_color_ex", "gc_set_stream", "gc_destroy",
           "gc_last_error", "gc_priorities", "gc_count_colors", "gc_version",
           "gc_trim", "gc_create_csr_dist", "gc_nccl_unique_id", "gc_create_csr_loopback"]


class GCError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"{STATUS.get(code, code)}: {msg}")
        self.code = code


class gc_options(ctypes.Structure):
    _fields_ = [("struct_size", ctypes.c_uint32), ("variant", ctypes.c_int32),
                ("seed", ctypes.c_uint64), ("flags", ctypes.c_uint32), ("mode", ctypes.c_int32),
                ("batch_rounds", ctypes.c_int32), ("thread_deg_max", ctypes.c_int32),
                ("hub_deg_min", ctypes.c_int32), ("reserved", ctypes.c_int32 * 7)]


class gc_stats(ctypes.Structure):
    _fields_ = [("struct_size", ctypes.c_uint32), ("mode_used", ctypes.c_int32),
                ("rounds", ctypes.c_int64), ("inner_iterations", ctypes.c_int64),
                ("n_colors", ctypes.c_int64), ("launches", ctypes.c_int64),
                ("ms", ctypes.c_double), ("frontier_sizes", ctypes.c_void_p),
                ("frontier_cap", ctypes.c_int64), ("kernel_ms", ctypes.c_double * 4),
                ("kernel_launches", ctypes.c_int64 * 4), ("kernel_bytes", ctypes.c_int64 * 4),
                ("visits", ctypes.c_int64), ("launch_us", ctypes.c_void_p),
                ("launch_cap", ctypes.c_int64), ("round_stats", ctypes.c_void_p),
                ("round_stats_cap", ctypes.c_int64)]


_lib = None


def lib():
    """Load libgc.so (built by __graft_entry__.build() / build.py). Raises if absent."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"{LIB_PATH} is missing: run `python -m "
                              "paper_conf_ipps_osamatybo19_b200.build` (no CPU fallback exists)")
        # torch loads the CUDA runtime / NCCL that libgc links against
        import torch  # noqa: F401
        L = ctypes.CDLL(LIB_PATH, mode=ctypes.RTLD_GLOBAL)
        i64, u64, i32, u32, P = (ctypes.c_int64, ctypes.c_uint64, ctypes.c_int32,
                                 ctypes.c_uint32, ctypes.c_void_p)
        L.gc_create_csr.argtypes = [i64, i64, P, P, u32, ctypes.POINTER(P)]
        L.gc_create_csr.restype = ctypes.c_int
        L.gc_color.argtypes, L.gc_color.restype = [P, u64, i32, P], i64
        L.gc_color_ex.argtypes = [P, ctypes.POINTER(gc_options), P, ctypes.POINTER(gc_stats)]
        L.gc_color_ex.restype = i64
        L.gc_set_stream.argtypes, L.gc_set_stream.restype = [P, P], ctypes.c_int
        L.gc_destroy.argtypes, L.gc_destroy.restype = [P], None
        L.gc_last_error.argtypes, L.gc_last_error.restype = [], ctypes.c_char_p
        L.gc_priorities.argtypes, L.gc_priorities.restype = [u64, i32, i64, i64, P], ctypes.c_int
        L.gc_count_colors.argtypes, L.gc_count_colors.restype = [P, i64], i64
        L.gc_version.argtypes, L.gc_version.restype = [], ctypes.c_char_p
        L.gc_trim.argtypes, L.gc_trim.restype = [], ctypes.c_int
        L.gc_create_csr_dist.argtypes = [i64, i64, i64, i64, P, P, P, ctypes.c_int, ctypes.c_int,
                                         u32, ctypes.POINTER(P)]
        L.gc_create_csr_dist.restype = ctypes.c_int
        L.gc_nccl_unique_id.argtypes, L.gc_nccl_unique_id.restype = [P], ctypes.c_int
        L.gc_create_csr_loopback.argtypes = [i64, i64, P, P, ctypes.c_int, u32, ctypes.POINTER(P)]
        L.gc_create_csr_loopback.restype = ctypes.c_int
        _lib = L
    return _lib


def last_error() -> str:
    return lib().gc_last_error().decode()


def _check(rc: int) -> int:
    if rc < 0:
        raise GCError(rc, last_error())
    return rc


def _numel(t) -> int:
    return int(t.numel()) if hasattr(t, "numel") else int(t.size)


def _need(t, count: int, what: str) -> None:
    """The C side reads / writes `count` elements of `t`: a shorter buffer
    would be an out-of-bounds access, so it is rejected here."""
    if t is not None and _numel(t) < count:
        raise ValueError(f"{what}: {_numel(t)} elements, {count} needed")


def _ptr(t, dtypes):
    """Pointer of a contiguous torch tensor or numpy array with an allowed dtype."""
    if t is None:
        return None
    if hasattr(t, "data_ptr"):
        if not t.is_contiguous():
            raise ValueError("tensor must be contiguous")
        if str(t.dtype).replace("torch.", "") not in dtypes:
            raise TypeError(f"dtype {t.dtype} not in {dtypes}")
        return ctypes.c_void_p(t.data_ptr()) if t.numel() else None
    import numpy as np
    a = t
    if not a.flags["C_CONTIGUOUS"]:
        raise ValueError("array must be C-contiguous")
    if a.dtype.name not in dtypes:
        raise TypeError(f"dtype {a.dtype} not in {dtypes}")
    return a.ctypes.data_as(ctypes.c_void_p) if a.size else None


@dataclass
class ColorStats:
    mode_used: int
    rounds: int
    inner_iterations: int
    n_colors: int
    launches: int
    ms: float
    frontier_sizes: list
    kernel_ms: list
    kernel_launches: list
    kernel_bytes: list
    visits: int
    launch_us: list
    round_stats: list


class Graph:
    """Owning wrapper of a gc_graph handle (gc_create_csr / gc_destroy)."""

    def __init__(self, n: int, row_offsets, col_indices, flags: int = 0):
        self._h = ctypes.c_void_p()
        self.n = int(n)
        self.nnz = _numel(col_indices)
        self.out_len = self.n  # colours written by color() (dist handles: see dist_graph)
        if self.n >= 0 and _numel(row_offsets) != self.n + 1:
            raise ValueError(f"row_offsets: {_numel(row_offsets)} elements, n + 1 = {self.n + 1} needed")
        self._keep = (row_offsets, col_indices) if flags & BORROW_DEVICE else None
        _check(lib().gc_create_csr(self.n, self.nnz, _ptr(row_offsets, ("int64",)),
                                   _ptr(col_indices, ("int32", "uint32")), flags,
                                   ctypes.byref(self._h)))

    @classmethod
    def _from_handle(cls, h, n, nnz, keep=None):
        obj = cls.__new__(cls)
        obj._h, obj.n, obj.nnz, obj._keep = h, n, nnz, keep
        obj.out_len = n
        return obj

    def set_stream(self, stream) -> None:
        """stream: a torch.cuda.Stream, a raw cudaStream_t int, or None (default)."""
        raw = 0 if stream is None else int(getattr(stream, "cuda_stream", stream))
        _check(lib().gc_set_stream(self._h, ctypes.c_void_p(raw)))

    def color(self, seed: int = 1, variant: int = MAXMIN, out=None, *, flags: int = 0,
              mode: int = MODE_AUTO, batch_rounds: int = 0, thread_deg_max: int = 0,
              hub_deg_min: int = 0, stats: bool = False, frontier_cap: int = 0,
              trace_cap: int = 0):
        """Colour the graph.  `out`: int32 tensor/array of n entries on host or
        device (allocated on the host if None).  Returns (out, n_colors) or
        (out, n_colors, ColorStats) with stats=True."""
        need = self.local_len if (flags & OUT_LOCAL_SLICE and hasattr(self, "local_len")) else self.out_len
        if out is None:
            import torch
            out = torch.empty(need, dtype=torch.int32)
        _need(out, need, "out")
        o = gc_options()
        o.struct_size = ctypes.sizeof(gc_options)
        o.variant, o.seed, o.flags, o.mode = variant, seed, flags, mode
        o.batch_rounds, o.thread_deg_max, o.hub_deg_min = batch_rounds, thread_deg_max, hub_deg_min
        st = gc_stats()
        st.struct_size = ctypes.sizeof(gc_stats)
        fs = None
        if frontier_cap:
            fs = (ctypes.c_int64 * frontier_cap)()
            st.frontier_sizes = ctypes.cast(fs, ctypes.c_void_p)
            st.frontier_cap = frontier_cap
        lu = rs = None
        if trace_cap:
            lu = (ctypes.c_float * (4 * trace_cap))()
            rs = (ctypes.c_int64 * (16 * trace_cap))()
            st.launch_us, st.launch_cap = ctypes.cast(lu, ctypes.c_void_p), 4 * trace_cap
            st.round_stats, st.round_stats_cap = ctypes.cast(rs, ctypes.c_void_p), trace_cap
        r = _check(lib().gc_color_ex(self._h, ctypes.byref(o), _ptr(out, ("int32",)),
                                     ctypes.byref(st)))
        if stats:
            nk = list(fs[: min(frontier_cap, st.rounds)]) if fs is not None else []
            return out, r, ColorStats(st.mode_used, st.rounds, st.inner_iterations, st.n_colors,
                                      st.launches, st.ms, nk, list(st.kernel_ms),
                                      list(st.kernel_launches), list(st.kernel_bytes), st.visits,
                                      list(lu[: min(4 * trace_cap, 4 * st.rounds + 8)]) if lu else [],
                                      list(rs[: min(16 * trace_cap, 16 * st.rounds)]) if rs else [])
        return out, r

    def close(self) -> None:
        if self._h:
            lib().gc_destroy(self._h)
            self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()


def loopback_graph(n: int, row_offsets, col_indices, parts: int, flags: int = 0) -> Graph:
    """The partitioned (multi-GPU) algorithm with `parts` partitions on this GPU."""
    h = ctypes.c_void_p()
    nnz = _numel(col_indices)
    if _numel(row_offsets) != n + 1:
        raise ValueError(f"row_offsets: {_numel(row_offsets)} elements, n + 1 = {n + 1} needed")
    _check(lib().gc_create_csr_loopback(n, nnz, _ptr(row_offsets, ("int64",)),
                                        _ptr(col_indices, ("int32", "uint32")), parts, flags,
                                        ctypes.byref(h)))
    return Graph._from_handle(h, n, nnz)


def nccl_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(128)
    _check(lib().gc_nccl_unique_id(buf))
    return buf.raw


def dist_graph(n_global: int, v_begin: int, v_end: int, row_offsets_local, col_indices_global,
               unique_id: bytes, rank: int, world: int, flags: int = 0) -> Graph:
    """A rank's share of a 1D-partitioned graph (collective over `world` ranks)."""
    h = ctypes.c_void_p()
    nnz = _numel(col_indices_global)
    if _numel(row_offsets_local) != v_end - v_begin + 1:
        raise ValueError(f"row_offsets_local: {_numel(row_offsets_local)} elements, "
                         f"{v_end - v_begin + 1} needed")
    uid = ctypes.create_string_buffer(bytes(unique_id), 128)
    _check(lib().gc_create_csr_dist(n_global, v_begin, v_end, nnz,
                                    _ptr(row_offsets_local, ("int64",)),
                                    _ptr(col_indices_global, ("int32", "uint32")), uid, rank,
                                    world, flags, ctypes.byref(h)))
    g = Graph._from_handle(h, n_global, nnz,
                           keep=(row_offsets_local, col_indices_global) if flags & BORROW_DEVICE
                           else None)
    g.local_len = v_end - v_begin  # GC_OUT_LOCAL_SLICE writes the owned range only
    return g


def color(n, row_offsets, col_indices, seed=1, variant=MAXMIN, out=None, **kw):
    """One-shot create + colour + destroy (the e2e path of bench.py)."""
    with Graph(n, row_offsets, col_indices) as g:
        return g.color(seed, variant, out, **kw)


def priorities(seed: int, j: int, v_begin: int, count: int, out):
    """a0: out[i] = p_j(v_begin + i) computed on the GPU (host or device out)."""
    _need(out, count, "out")
    _check(lib().gc_priorities(seed, j, v_begin, count, _ptr(out, ("int32", "uint32"))))
    return out


def count_colors(colors) -> int:
    n = colors.numel() if hasattr(colors, "numel") else colors.size
    return _check(lib().gc_count_colors(_ptr(colors, ("int32",)), n))


def version() -> str:
    return lib().gc_version().decode()


def trim() -> None:
    """Return the library's cached device / pinned blocks to the driver."""
    _check(lib().gc_trim())
