"""CPU oracle for the IS colouring sweep (Alg.1-5) -- TEST INFRASTRUCTURE.

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl
reference legs may import this package.  The product path
(paper_conf_ipps_osamatybo19_b200) never imports it and shares no code with
it.  The arithmetic lives in oracle.c (plain C + OpenMP); this module only
compiles it (gcc) and marshals numpy/torch arrays through ctypes.

Parity status per function:
  priority            pinned (SMHasher fmix32 vectors, inverse, distinctness)
  color_maxmin (H>=1) pinned (literal in-place Alg.5 transcription, closed forms,
                      certificate, brute-force chi)
  color_luby          pinned (descending-priority greedy closed form, Python JP)
  color_greedy        pinned (Delta+1, closed forms)
  color_is_alg2       pinned (golden, longest-decreasing-path DP, properness)
  color_jp_alg4       pinned (golden, K_n / edgeless closed forms, first-free
                      property per frontier, properness)
  color_hash_is       pinned (golden at T = 0/1/4, K_n closed form, row-order
                      invariance, properness, progress bound R <= 2n+2)
  ldf (all of the above but Hash IS, reading R21)
                      pinned (literal Alg.5 with (degree, weight) tuple keys,
                      LDF greedy = JP closed form, longest-path DP, star and
                      regular-graph closed forms, certificates with mutations)
  paper-value parity  unpinned: the paper prints no colour count or worked
                      example for any variant (Fig.1b/3 unreadable).
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import time

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
UNCOLORED = 0xFFFFFFFF

_lib = None


def build(force: bool = False) -> str:
    """Compile oracle.c -> oracle/liboracle.so with gcc -O2 -fopenmp."""
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(_SRC):
        tmp = _LIB_PATH + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-fopenmp", "-fPIC", "-shared", "-Wall",
                               "-o", tmp, _SRC])
        os.replace(tmp, _LIB_PATH)
    return _LIB_PATH


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB_PATH)
        i64, u64, i32, u32 = ctypes.c_int64, ctypes.c_uint64, ctypes.c_int32, ctypes.c_uint32
        P = ctypes.c_void_p
        L.orc_fmix32.argtypes, L.orc_fmix32.restype = [u32], u32
        L.orc_hash_key.argtypes, L.orc_hash_key.restype = [u64, i32], u32
        L.orc_priority.argtypes, L.orc_priority.restype = [u64, i32, u32], u32
        L.orc_priorities.argtypes, L.orc_priorities.restype = [u64, i32, i64, P], None
        L.orc_color_maxmin.argtypes = [i64, P, P, u64, i32, P, P, i64, i64, i32]
        L.orc_color_maxmin.restype = i64
        L.orc_color_luby.argtypes, L.orc_color_luby.restype = [i64, P, P, u64, P, P, i32], i64
        L.orc_color_is_alg2.argtypes, L.orc_color_is_alg2.restype = [i64, P, P, u64, P, P, i32], i64
        L.orc_color_jp_alg4.argtypes, L.orc_color_jp_alg4.restype = [i64, P, P, u64, P, P, i32], i64
        L.orc_color_hash_is.argtypes = [i64, P, P, u64, i32, P, P]
        L.orc_color_hash_is.restype = i64
        L.orc_color_greedy.argtypes, L.orc_color_greedy.restype = [i64, P, P, P, P], i64
        L.orc_color_greedy_by_priority.argtypes = [i64, P, P, u64, P, i32]
        L.orc_color_greedy_by_priority.restype = i64
        L.orc_check_proper.argtypes, L.orc_check_proper.restype = [i64, P, P, P], i64
        L.orc_count_colors.argtypes, L.orc_count_colors.restype = [i64, P], i64
        L.orc_compact_colors.argtypes, L.orc_compact_colors.restype = [i64, P], i64
        L.orc_cert_maxmin.argtypes, L.orc_cert_maxmin.restype = [i64, P, P, u64, i32, P, i32], i64
        L.orc_cert_mex.argtypes, L.orc_cert_mex.restype = [i64, P, P, u64, P, i32], i64
        L.orc_num_threads.argtypes, L.orc_num_threads.restype = [], i32
        L.orc_set_threads.argtypes, L.orc_set_threads.restype = [i32], None
        _lib = L
    return _lib


def _csr(g):
    """(n, row_offsets int64 ndarray, col_indices uint32 ndarray) from a
    graphgen.Graph (torch) or a (n, ro, ci) tuple."""
    if isinstance(g, tuple):
        n, ro, ci = g
    else:
        n, ro, ci = g.n, g.row_offsets, g.col_indices
    if hasattr(ro, "cpu"):
        ro = ro.cpu().numpy()
    if hasattr(ci, "cpu"):
        ci = ci.cpu().numpy()
    ro = np.ascontiguousarray(ro, dtype=np.int64)
    ci = np.ascontiguousarray(ci).view(np.uint32) if np.asarray(ci).dtype in (np.int32, np.uint32) \
        else np.ascontiguousarray(ci, dtype=np.uint32)
    return int(n), ro, ci


def _p(a):
    return a.ctypes.data_as(ctypes.c_void_p) if a is not None and a.size else None


def _pp(a):
    return a.ctypes.data_as(ctypes.c_void_p)


def fmix32(x: int) -> int:
    return int(lib().orc_fmix32(x & 0xFFFFFFFF))


def hash_key(seed: int, j: int) -> int:
    return int(lib().orc_hash_key(seed, j))


def priority(seed: int, j: int, v: int) -> int:
    return int(lib().orc_priority(seed, j, v))


def priorities(seed: int, j: int, n: int) -> np.ndarray:
    out = np.empty(max(n, 1), dtype=np.uint32)
    lib().orc_priorities(seed, j, n, _pp(out))
    return out[:n]


class OracleError(RuntimeError):
    pass


def color_maxmin(g, seed: int, H: int = 1, max_rounds: int = 1 << 40,
                 with_stats: bool = False, ldf: bool = False):
    """Max-min (H=1) / multi-hash (H>1) IS colouring, Alg.1 + Alg.5 with snapshot
    semantics. Returns uint32 raw colours (and (rounds, N_k list) if with_stats).
    ldf: priorities (degree, weight), largest degree first (R21)."""
    n, ro, ci = _csr(g)
    C = np.empty(max(n, 1), dtype=np.uint32)
    cap = 1 << 16
    nk = np.zeros(cap, dtype=np.int64)
    r = lib().orc_color_maxmin(n, _pp(ro), _p(ci), seed, H, _pp(C), _pp(nk), cap, max_rounds,
                               int(ldf))
    if r < 0:
        raise OracleError(f"orc_color_maxmin failed: {r}")
    C = C[:n]
    if with_stats:
        return C, int(r), nk[: min(int(r), cap)].tolist()
    return C


def color_luby(g, seed: int, with_stats: bool = False, ldf: bool = False):
    """Luby MIS colouring, Alg.2 outer + Alg.3 inner loop, fixed weights."""
    n, ro, ci = _csr(g)
    C = np.empty(max(n, 1), dtype=np.uint32)
    inner = np.zeros(1, dtype=np.int64)
    r = lib().orc_color_luby(n, _pp(ro), _p(ci), seed, _pp(C), _pp(inner), int(ldf))
    if r < 0:
        raise OracleError(f"orc_color_luby failed: {r}")
    if with_stats:
        return C[:n], int(r), int(inner[0])
    return C[:n]


def _alg2(fn, g, seed, with_stats, ldf=False):
    n, ro, ci = _csr(g)
    C = np.empty(max(n, 1), dtype=np.uint32)
    rounds = np.zeros(1, dtype=np.int64)
    r = fn(n, _pp(ro), _p(ci), seed, _pp(C), _pp(rounds), int(ldf))
    if r < 0:
        raise OracleError(f"{fn.__name__} failed: {r}")
    return (C[:n], int(rounds[0])) if with_stats else C[:n]


def color_is_alg2(g, seed: int, with_stats: bool = False, ldf: bool = False):
    """Max-only IS colouring, Alg.2 as written (colour = iteration)."""
    return _alg2(lib().orc_color_is_alg2, g, seed, with_stats, ldf)


def color_jp_alg4(g, seed: int, with_stats: bool = False, ldf: bool = False):
    """GraphBLAS Jones-Plassmann, Alg.2 with Alg.4's frontier colour."""
    return _alg2(lib().orc_color_jp_alg4, g, seed, with_stats, ldf)


def color_hash_is(g, seed: int, table: int, with_stats: bool = False):
    """Hash IS colouring, Alg.6 made deterministic (R16-R20), table size T."""
    n, ro, ci = _csr(g)
    C = np.empty(max(n, 1), dtype=np.uint32)
    rounds = np.zeros(1, dtype=np.int64)
    r = lib().orc_color_hash_is(n, _pp(ro), _p(ci), seed, table, _pp(C), _pp(rounds))
    if r < 0:
        raise OracleError(f"orc_color_hash_is failed: {r}")
    return (C[:n], int(r), int(rounds[0])) if with_stats else C[:n]


def color_greedy(g, order=None):
    """Sequential first-fit greedy (natural order unless `order` is given)."""
    n, ro, ci = _csr(g)
    C = np.empty(max(n, 1), dtype=np.uint32)
    o = None if order is None else np.ascontiguousarray(order, dtype=np.int64)
    r = lib().orc_color_greedy(n, _pp(ro), _p(ci), _p(o) if o is not None else None, _pp(C))
    if r < 0:
        raise OracleError(f"orc_color_greedy failed: {r}")
    return C[:n]


def color_greedy_by_priority(g, seed: int, ldf: bool = False):
    """First-fit greedy in descending p_0 order (closed form of Luby, R10)."""
    n, ro, ci = _csr(g)
    C = np.empty(max(n, 1), dtype=np.uint32)
    r = lib().orc_color_greedy_by_priority(n, _pp(ro), _p(ci), seed, _pp(C), int(ldf))
    if r < 0:
        raise OracleError(f"orc_color_greedy_by_priority failed: {r}")
    return C[:n]


def check_proper(g, C) -> int:
    n, ro, ci = _csr(g)
    C = np.ascontiguousarray(C, dtype=np.uint32)
    return int(lib().orc_check_proper(n, _pp(ro), _p(ci), _p(C)))


def count_colors(C) -> int:
    C = np.ascontiguousarray(C, dtype=np.uint32)
    return int(lib().orc_count_colors(C.size, _p(C)))


def compact_colors(C) -> np.ndarray:
    C = np.array(C, dtype=np.uint32, copy=True)
    lib().orc_compact_colors(C.size, _p(C))
    return C


def cert_maxmin(g, seed: int, H: int, C, ldf: bool = False) -> int:
    n, ro, ci = _csr(g)
    C = np.ascontiguousarray(C, dtype=np.uint32)
    return int(lib().orc_cert_maxmin(n, _pp(ro), _p(ci), seed, H, _p(C), int(ldf)))


def cert_mex(g, seed: int, C, ldf: bool = False) -> int:
    n, ro, ci = _csr(g)
    C = np.ascontiguousarray(C, dtype=np.uint32)
    return int(lib().orc_cert_mex(n, _pp(ro), _p(ci), seed, _p(C), int(ldf)))


def num_threads() -> int:
    return int(lib().orc_num_threads())


def set_threads(t: int) -> None:
    lib().orc_set_threads(t)


def reference_color(g, seed: int, variant: str, H: int = 1):
    """Dispatch used by bench.py's reference arm: variant in
    {'maxmin', 'multihash', 'luby'}; returns (colors, seconds)."""
    t0 = time.perf_counter()
    if variant == "luby":
        C = color_luby(g, seed)
    else:
        C = color_maxmin(g, seed, H if variant == "multihash" else 1)
    return C, time.perf_counter() - t0
