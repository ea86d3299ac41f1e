"""Host-side logic of the 1D vertex partition with
torch.distributed over gloo, world size 2, on the CPU: ranges, per-rank rows
built from the shared pair stream, the nnz reduction and the NCCL-id broadcast.
The per-round exchange itself is tested bit-exactly on one GPU through the
loopback transport (tests/test_gpu_parity.py::test_loopback_partitions)."""
import os
import socket

import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import graphgen as G
from paper_conf_ipps_osamatybo19_b200 import dist as gdist


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        scale = 10
        g = G.rmat(scale, 16, seed=3)
        n, v0, v1, ro, ci = gdist.rmat_local(scale, 16, 3, rank, world, "cpu")
        ro_ref, ci_ref = gdist.local_rows(g, v0, v1)
        ok_rows = torch.equal(ro, ro_ref) and torch.equal(ci, ci_ref)
        nnz = torch.tensor([ci.numel()], dtype=torch.int64)
        dist.all_reduce(nnz)
        uid = gdist.broadcast_unique_id(bytes(range(128)) if rank == 0 else None)
        q.put((rank, ok_rows, int(nnz.item()) == g.nnz, uid == bytes(range(128)), v0, v1, n))
    finally:
        dist.destroy_process_group()


def test_partition_host_logic_world2():
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=240) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    assert [r[0] for r in res] == [0, 1]
    assert all(r[1] for r in res), "rank rows differ from the global CSR slice"
    assert all(r[2] for r in res), "nnz reduction differs"
    assert all(r[3] for r in res), "unique id broadcast"
    n = res[0][6]
    assert res[0][4] == 0 and res[0][5] == res[1][4] and res[1][5] == n


@pytest.mark.parametrize("n,world", [(10, 3), (1 << 20, 8), (7, 8), (0, 2)])
def test_split_range_covers(n, world):
    ranges = [gdist.split_range(n, world, r) for r in range(world)]
    assert ranges[0][0] == 0 and ranges[-1][1] == n
    for (a0, a1), (b0, b1) in zip(ranges, ranges[1:]):
        assert a1 == b0 and a0 <= a1


def test_local_csr_from_pairs_matches_global():
    g = G.erdos_renyi(3000, 20000, seed=4)
    us, vs = [], []
    key = G._stream_key(4, 0xE5)
    e = torch.arange(20000, dtype=torch.int64)
    us.append(G._uniform_below(G.splitmix64((2 * e) ^ key), 3000))
    vs.append(G._uniform_below(G.splitmix64((2 * e + 1) ^ key), 3000))
    for v0, v1 in ((0, 1000), (1000, 2999), (2999, 3000)):
        ro, ci = gdist.local_csr_from_pairs(3000, v0, v1, us, vs)
        ro_ref, ci_ref = gdist.local_rows(g, v0, v1)
        assert torch.equal(ro, ro_ref) and torch.equal(ci, ci_ref)
