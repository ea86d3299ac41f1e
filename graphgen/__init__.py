"""Seeded synthetic graph generators shared by the oracle tests and the CUDA path.

This module holds NONE of the colouring method's arithmetic: it only builds
undirected CSR graphs (symmetrised, self-loops dropped, duplicates removed),
the input preparation the paper describes for its datasets
("All datasets have been converted to undirected graphs, and self-loops and
duplicated edges are removed", Sec. V-A).

Every random number comes from a counter-based splitmix64 stream, so a graph is
a pure function of (generator, size, seed) and is identical whether it is built
on the CPU or on a CUDA device (all arithmetic is torch int64 with explicit
masks for the logical shifts; int64 multiply wraps mod 2^64 on both devices).

Workload shapes (SURVEY.md §8(d) "Concrete inputs", BASELINE.json configs):
  cfg1  grid2d(64, 64)                      2D 5-point grid
  cfg2  erdos_renyi(2**20, 8 * 2**20)       ER G(n, M), avg degree 16
  cfg3  mesh3d(128, 128, 128)               3D 7-point mesh (FEM-like)
  cfg4  rmat(24, 16)                        Graph500 Kronecker A,B,C=.57,.19,.19
  cfg5  rmat(27, 16)                        same, partitioned across GPUs
  N1    rgg(scale)                          DIMACS10-style random geometric graph,
                                            r = 0.55 sqrt(ln n / n) (Table I rgg rows,
                                            P:L699-708)
"""
from __future__ import annotations

import math
from dataclasses import dataclass, field

import torch

_M64 = (1 << 64) - 1


def _s64(x: int) -> int:
    """Reinterpret an unsigned 64-bit constant as a signed int64 literal."""
    x &= _M64
    return x - (1 << 64) if x >= (1 << 63) else x


_GOLD = _s64(0x9E3779B97F4A7C15)
_MIX1 = _s64(0xBF58476D1CE4E5B9)
_MIX2 = _s64(0x94D049BB133111EB)


def _srl(x: torch.Tensor, k: int) -> torch.Tensor:
    """Logical right shift of int64 bit patterns."""
    return (x >> k) & ((1 << (64 - k)) - 1)


def splitmix64(x: torch.Tensor) -> torch.Tensor:
    """splitmix64 finaliser applied to counters x (int64 bit patterns)."""
    z = x + _GOLD
    z = (z ^ _srl(z, 30)) * _MIX1
    z = (z ^ _srl(z, 27)) * _MIX2
    return z ^ _srl(z, 31)


def splitmix64_int(x: int) -> int:
    """Python-int reference of splitmix64 (used for stream keys)."""
    z = (x + 0x9E3779B97F4A7C15) & _M64
    z = ((z ^ (z >> 30)) * 0xBF58476D1CE4E5B9) & _M64
    z = ((z ^ (z >> 27)) * 0x94D049BB133111EB) & _M64
    return z ^ (z >> 31)


def _stream_key(seed: int, tag: int) -> int:
    return _s64(splitmix64_int((seed * 0x100000001B3 + tag) & _M64))


@dataclass
class Graph:
    """Undirected CSR graph: row_offsets int64[n+1], col_indices int32[nnz]
    (vertex ids < 2^31 here; the C ABI reads them as uint32)."""

    n: int
    row_offsets: torch.Tensor
    col_indices: torch.Tensor
    name: str = ""
    meta: dict = field(default_factory=dict)

    @property
    def nnz(self) -> int:
        return int(self.col_indices.numel())

    def to(self, device) -> "Graph":
        return Graph(self.n, self.row_offsets.to(device), self.col_indices.to(device),
                     self.name, dict(self.meta))

    def degrees(self) -> torch.Tensor:
        return self.row_offsets[1:] - self.row_offsets[:-1]


def csr_from_pairs(n: int, u: torch.Tensor, v: torch.Tensor, name: str = "",
                   meta: dict | None = None) -> Graph:
    """Symmetrise, drop self-loops, dedup, sort rows ascending -> CSR."""
    device = u.device
    u = u.to(torch.int64)
    v = v.to(torch.int64)
    keep = u != v
    u, v = u[keep], v[keep]
    keys = torch.cat([u * n + v, v * n + u])
    del u, v, keep
    keys = torch.unique(keys, sorted=True)
    rows = keys // n
    cols = (keys - rows * n).to(torch.int32)
    del keys
    counts = torch.bincount(rows, minlength=n)
    del rows
    ro = torch.zeros(n + 1, dtype=torch.int64, device=device)
    ro[1:] = torch.cumsum(counts, 0)
    return Graph(n, ro, cols, name, dict(meta or {}))


def csr_from_lists(n: int, edges, name: str = "") -> Graph:
    """Tiny hand-written graphs: edges is an iterable of (u, v)."""
    edges = list(edges)
    if not edges:
        return Graph(n, torch.zeros(n + 1, dtype=torch.int64),
                     torch.zeros(0, dtype=torch.int32), name)
    t = torch.tensor(edges, dtype=torch.int64)
    return csr_from_pairs(n, t[:, 0], t[:, 1], name)


def grid2d(rows: int, cols: int, device="cpu") -> Graph:
    """2D 5-point grid, v = i*cols + j, 4-neighbour, no wrap (cfg1)."""
    n = rows * cols
    idx = torch.arange(n, dtype=torch.int64, device=device)
    i, j = idx // cols, idx % cols
    us, vs = [], []
    m = j + 1 < cols
    us.append(idx[m]); vs.append(idx[m] + 1)
    m = i + 1 < rows
    us.append(idx[m]); vs.append(idx[m] + cols)
    return csr_from_pairs(n, torch.cat(us), torch.cat(vs), f"grid2d_{rows}x{cols}",
                          {"kind": "grid2d", "rows": rows, "cols": cols})


def mesh3d(nx: int, ny: int, nz: int, device="cpu") -> Graph:
    """3D 7-point mesh, v = (i*ny + j)*nz + l, 6-neighbour, no wrap (cfg3)."""
    n = nx * ny * nz
    idx = torch.arange(n, dtype=torch.int64, device=device)
    l = idx % nz
    j = (idx // nz) % ny
    i = idx // (ny * nz)
    us, vs = [], []
    for cond, step in ((l + 1 < nz, 1), (j + 1 < ny, nz), (i + 1 < nx, ny * nz)):
        us.append(idx[cond]); vs.append(idx[cond] + step)
    return csr_from_pairs(n, torch.cat(us), torch.cat(vs), f"mesh3d_{nx}x{ny}x{nz}",
                          {"kind": "mesh3d", "dims": [nx, ny, nz]})


def _uniform_below(h: torch.Tensor, n: int) -> torch.Tensor:
    """Map 64-bit hashes to [0, n): power-of-two n takes the low bits,
    otherwise the non-negative 63-bit value modulo n."""
    if n & (n - 1) == 0:
        return h & (n - 1)
    return _srl(h, 1) % n


def erdos_renyi(n: int, m_pairs: int, seed: int = 1, device="cpu",
                chunk: int = 1 << 24) -> Graph:
    """G(n, M): pair e = (h(2e) mod n, h(2e+1) mod n), h = splitmix64 keyed by
    seed; loops dropped, symmetrised, deduplicated (cfg2: n=2^20, M=8n)."""
    key = _stream_key(seed, 0xE5)
    us, vs = [], []
    for s in range(0, m_pairs, chunk):
        e = torch.arange(s, min(s + chunk, m_pairs), dtype=torch.int64, device=device)
        us.append(_uniform_below(splitmix64((2 * e) ^ key), n))
        vs.append(_uniform_below(splitmix64((2 * e + 1) ^ key), n))
    return csr_from_pairs(n, torch.cat(us), torch.cat(vs), f"er_n{n}_m{m_pairs}",
                          {"kind": "er", "n": n, "m_pairs": m_pairs, "seed": seed})


def _label_permutation(x: torch.Tensor, scale: int, seed: int) -> torch.Tensor:
    """Seeded bijection on [0, 2^scale): 3 rounds of (odd multiply + add) mod 2^s
    followed by an in-word xorshift; each step is invertible on s-bit words."""
    if scale == 0:
        return x
    mask = (1 << scale) - 1
    for r in range(3):
        a = splitmix64_int((seed * 0x51ED27 + 0x9E37 + r) & _M64)
        mul = (a | 1) & mask
        add = (a >> 32) & mask
        x = (x * mul + add) & mask
        x = x ^ (x >> max(1, scale // 2))
    return x


def rmat_pairs(scale: int, edge_factor: int = 16, seed: int = 1, device="cpu",
               a: float = 0.57, b: float = 0.19, c: float = 0.19,
               begin: int = 0, end: int | None = None,
               chunk: int = 1 << 22):
    """Yield (u, v) int64 chunks of Graph500 Kronecker pairs [begin, end).

    Pair e, level l draws a 32-bit uniform r (two levels per splitmix64 call)
    and picks quadrant (0,0) if r < A, (0,1) if r < A+B, (1,0) if r < A+B+C,
    else (1,1). Labels then go through a seeded bijection of [0, 2^scale)."""
    m = edge_factor << scale
    end = m if end is None else end
    ta = int(a * 2**32)
    tab = int((a + b) * 2**32)
    tabc = int((a + b + c) * 2**32)
    key = _stream_key(seed, 0x4D)
    nlev2 = (scale + 1) // 2
    for s in range(begin, end, chunk):
        e = torch.arange(s, min(s + chunk, end), dtype=torch.int64, device=device)
        u = torch.zeros_like(e)
        v = torch.zeros_like(e)
        base = e * nlev2
        for l2 in range(nlev2):
            h = splitmix64((base + l2) ^ key)
            for half in range(2):
                lev = 2 * l2 + half
                if lev >= scale:
                    break
                r = _srl(h, 32) if half == 0 else (h & 0xFFFFFFFF)
                ubit = (r >= tab).to(torch.int64)
                vbit = ((r >= ta) & (r < tab)).to(torch.int64) | (r >= tabc).to(torch.int64)
                u = u | (ubit << lev)
                v = v | (vbit << lev)
        yield _label_permutation(u, scale, seed), _label_permutation(v, scale, seed)


def rmat(scale: int, edge_factor: int = 16, seed: int = 1, device="cpu", pieces: int = 1) -> Graph:
    """R-MAT / Graph500 Kronecker graph, symmetrised (cfg4: s24, cfg5: s27).

    pieces > 1 builds the same CSR row range by row range (each range keeps
    the pairs touching it from a fresh pass over the counter-based pair
    stream), so peak memory is about 1/pieces of the one-shot build (cfg5)."""
    n = 1 << scale
    meta = {"kind": "rmat", "scale": scale, "edge_factor": edge_factor, "seed": seed}
    name = f"rmat_s{scale}_ef{edge_factor}"
    if pieces <= 1:
        us, vs = [], []
        for u, v in rmat_pairs(scale, edge_factor, seed, device):
            us.append(u); vs.append(v)
        return csr_from_pairs(n, torch.cat(us), torch.cat(vs), name, meta)
    step = (n + pieces - 1) // pieces
    ros, cis, base = [], [], 0
    for v0 in range(0, n, step):
        v1 = min(n, v0 + step)
        keys = []
        for u, v in rmat_pairs(scale, edge_factor, seed, device):
            keep = u != v
            u, v = u[keep], v[keep]
            for a, b in ((u, v), (v, u)):
                m = (a >= v0) & (a < v1)
                keys.append((a[m] - v0) * n + b[m])
        k = torch.unique(torch.cat(keys), sorted=True)
        del keys
        rows = k // n
        cis.append((k - rows * n).to(torch.int32))
        del k
        ro = torch.cumsum(torch.bincount(rows, minlength=v1 - v0), 0) + base
        del rows
        ros.append(ro)
        base = int(ro[-1]) if ro.numel() else base
    ro = torch.cat([torch.zeros(1, dtype=torch.int64, device=device)] + ros)
    return Graph(n, ro, torch.cat(cis), name, meta)


def rgg(scale: int, seed: int = 1, device="cpu", radius_coef: float = 0.55) -> Graph:
    """Random geometric graph in the unit square (DIMACS10 rgg_n_2_<scale>):
    n = 2^scale points, edge iff Euclidean distance < r = coef*sqrt(ln n / n).
    Coordinates are 53-bit uniforms from splitmix64; neighbour search buckets
    points into a grid of cell size >= r and compares the 3x3 cell block."""
    n = 1 << scale
    r = radius_coef * math.sqrt(math.log(n) / n)
    key = _stream_key(seed, 0x66)
    idx = torch.arange(n, dtype=torch.int64, device=device)
    x = _srl(splitmix64((2 * idx) ^ key), 11).to(torch.float64) * (2.0 ** -53)
    y = _srl(splitmix64((2 * idx + 1) ^ key), 11).to(torch.float64) * (2.0 ** -53)
    g = max(1, int(1.0 / r))
    cx = torch.clamp((x * g).to(torch.int64), max=g - 1)
    cy = torch.clamp((y * g).to(torch.int64), max=g - 1)
    cell = cx * g + cy
    order = torch.argsort(cell, stable=True)
    cell_sorted = cell[order]
    starts = torch.searchsorted(cell_sorted, torch.arange(g * g + 1, device=device))
    r2 = r * r
    us, vs = [], []
    for dx in (-1, 0, 1):
        for dy in (-1, 0, 1):
            nx_, ny_ = cx + dx, cy + dy
            ok = (nx_ >= 0) & (nx_ < g) & (ny_ >= 0) & (ny_ < g)
            src = idx[ok]
            ncell = (nx_ * g + ny_)[ok]
            lo, hi = starts[ncell], starts[ncell + 1]
            cnt = hi - lo
            total = int(cnt.sum())
            if total == 0:
                continue
            rep_src = torch.repeat_interleave(src, cnt)
            offs = torch.arange(total, device=device) - torch.repeat_interleave(
                torch.cumsum(cnt, 0) - cnt, cnt)
            dst = order[torch.repeat_interleave(lo, cnt) + offs]
            ddx = x[rep_src] - x[dst]
            ddy = y[rep_src] - y[dst]
            close = (ddx * ddx + ddy * ddy) < r2
            keep = close & (rep_src < dst)
            us.append(rep_src[keep]); vs.append(dst[keep])
    return csr_from_pairs(n, torch.cat(us), torch.cat(vs), f"rgg_n_2_{scale}",
                          {"kind": "rgg", "scale": scale, "seed": seed, "radius": r})


def random_graph(n: int, p: float, seed: int, device="cpu") -> Graph:
    """Small dense-ish random graph for exhaustive parity tests: each unordered
    pair (i<j) is an edge with probability p (hash-thresholded)."""
    if n <= 1:
        return Graph(n, torch.zeros(n + 1, dtype=torch.int64, device=device),
                     torch.zeros(0, dtype=torch.int32, device=device), f"rand_{n}")
    i = torch.arange(n, dtype=torch.int64, device=device)
    ii, jj = torch.meshgrid(i, i, indexing="ij")
    m = ii < jj
    ii, jj = ii[m], jj[m]
    key = _stream_key(seed, 0x77)
    h = _srl(splitmix64((ii * n + jj) ^ key), 11)
    keep = h < int(p * 2.0**53)
    return csr_from_pairs(n, ii[keep], jj[keep], f"rand_{n}_{p}_{seed}")


CONFIGS = {
    "cfg1": dict(desc="2D 5-point grid 64x64, max-min, seed=1"),
    "cfg2": dict(desc="Erdos-Renyi n=2^20 avg degree 16, Luby-MIS and max-min"),
    "cfg3": dict(desc="3D 7-point mesh 128^3, multi-hash H=4"),
    "cfg4": dict(desc="R-MAT scale 24, edge factor 16, max-min"),
    "cfg5": dict(desc="R-MAT scale 27, edge factor 16, partitioned across GPUs"),
}


def config_graph(name: str, device="cpu", seed: int = 1) -> Graph:
    if name == "cfg1":
        return grid2d(64, 64, device)
    if name == "cfg2":
        return erdos_renyi(1 << 20, 8 << 20, seed, device)
    if name == "cfg3":
        return mesh3d(128, 128, 128, device)
    if name == "cfg4":
        return rmat(24, 16, seed, device)
    if name == "cfg5":
        return rmat(27, 16, seed, device)
    raise KeyError(name)
