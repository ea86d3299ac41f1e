"""Host-side plumbing of the 1D vertex-range partition.

One process per GPU (torchrun); torch.distributed is the plumbing: it carries
the NCCL unique id from rank 0 and reduces sizes.  The per-round exchange runs
inside libgc (gc_create_csr_dist / gc_color) over NCCL.  This module only
decides ranges and builds each rank's rows; it has no colouring arithmetic.
"""
from __future__ import annotations

import torch

import graphgen as G


def split_range(n: int, world: int, rank: int) -> tuple[int, int]:
    """Equal contiguous ranges [v0, v1) (the last ones may be shorter)."""
    chunk = (n + world - 1) // world
    v0 = min(n, rank * chunk)
    return v0, min(n, v0 + chunk)


def local_rows(g: G.Graph, v0: int, v1: int) -> tuple[torch.Tensor, torch.Tensor]:
    """Rows [v0, v1) of a global CSR: rebased offsets and global column ids."""
    ro = g.row_offsets[v0:v1 + 1]
    base = int(ro[0])
    return (ro - base).contiguous(), g.col_indices[base:int(ro[-1])].contiguous()


def local_csr_from_pairs(n: int, v0: int, v1: int, us, vs) -> tuple[torch.Tensor, torch.Tensor]:
    """Rows [v0, v1) of the symmetrised, loop-free, deduplicated graph of the
    undirected pairs (us[i], vs[i]) -- without building the global CSR."""
    keys = []
    for u, v in zip(us, vs):
        keep = u != v
        u, v = u[keep], v[keep]
        for a, b in ((u, v), (v, u)):
            m = (a >= v0) & (a < v1)
            keys.append((a[m] - v0) * n + b[m])
    device = us[0].device if us else "cpu"
    k = torch.unique(torch.cat(keys)) if keys else torch.zeros(0, dtype=torch.int64, device=device)
    rows = k // n
    cols = (k - rows * n).to(torch.int32)
    ro = torch.zeros(v1 - v0 + 1, dtype=torch.int64, device=k.device)
    ro[1:] = torch.cumsum(torch.bincount(rows, minlength=v1 - v0), 0)
    return ro, cols


def rmat_local(scale: int, edge_factor: int, seed: int, rank: int, world: int, device):
    """This rank's rows of graphgen.rmat(scale, edge_factor, seed): every rank
    generates the same pair stream (counter-based) and keeps its own rows."""
    n = 1 << scale
    v0, v1 = split_range(n, world, rank)
    us, vs = [], []
    for u, v in G.rmat_pairs(scale, edge_factor, seed, device):
        m = ((u >= v0) & (u < v1)) | ((v >= v0) & (v < v1))
        us.append(u[m])
        vs.append(v[m])
    ro, ci = local_csr_from_pairs(n, v0, v1, us, vs)
    return n, v0, v1, ro, ci


def broadcast_unique_id(uid: bytes | None, group=None) -> bytes:
    """Rank 0's 128-byte NCCL unique id to every rank (torch.distributed)."""
    import torch.distributed as dist
    obj = [uid]
    dist.broadcast_object_list(obj, src=0, group=group)
    return obj[0]


def build_partitioned_rmat(scale: int, edge_factor: int, seed: int, rank: int, world: int,
                           device):
    """Build this rank's share of R-MAT(scale) on `device` and its gc handle.
    Returns (rows tuple, handle, n_global, nnz_global)."""
    import torch.distributed as dist

    import paper_conf_ipps_osamatybo19_b200 as gcb
    n, v0, v1, ro, ci = rmat_local(scale, edge_factor, seed, rank, world, device)
    nnz = torch.tensor([ci.numel()], dtype=torch.int64, device=device)
    dist.all_reduce(nnz)
    uid = broadcast_unique_id(gcb.nccl_unique_id() if rank == 0 else None)
    h = gcb.dist_graph(n, v0, v1, ro, ci, uid, rank, world, flags=gcb.BORROW_DEVICE)
    return (ro, ci), h, n, int(nnz.item())
