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


# ----------------------------------------------------------------------------
# The partitioned COUNT protocol (csrc/gc_dist_count.cu) as a
# plain model over gloo, world size 2: owned counts, ghost rows, per-round
# all-gather of coloured pairs.  Checks the protocol (what each rank must
# know each round) against the oracle; the CUDA kernels implementing it are
# checked bit-exactly on the GPU (loopback and NCCL tests).
def _count_protocol_worker(rank, world, port, q, scale, seed):
    import numpy as np

    import oracle as O
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        g = G.rmat(scale, 8, seed=seed)
        n = g.n
        v0, v1 = gdist.split_range(n, world, rank)
        ro, ci = (t.numpy() for t in gdist.local_rows(g, v0, v1))
        p = O.priorities(seed, 0, n).astype(np.int64)
        nl = v1 - v0
        hi = np.zeros(nl, dtype=np.int64)
        lo = np.zeros(nl, dtype=np.int64)
        ghost = {}
        for lv in range(nl):
            row = ci[ro[lv]:ro[lv + 1]].astype(np.int64)
            hi[lv] = int((p[row] > p[v0 + lv]).sum())
            lo[lv] = len(row) - hi[lv]
            for u in row:
                if not v0 <= u < v1:
                    ghost.setdefault(int(u), []).append(lv)
        UNC, NEVER = 0xFFFFFFFF, 1 << 62
        C = np.full(n, UNC, dtype=np.uint32)
        Z = np.full(nl, NEVER, dtype=np.int64)
        S = [(lv, lo[lv] == 0) for lv in range(nl) if hi[lv] == 0 or lo[lv] == 0]
        k, remaining = 0, n
        while remaining > 0:
            nxt = []

            def dec(pv, lw):
                nonlocal nxt
                if pv > p[v0 + lw]:
                    hi[lw] -= 1
                    side, other, lo_side = hi[lw], lo[lw], False
                else:
                    lo[lw] -= 1
                    side, other, lo_side = lo[lw], hi[lw], True
                assert side >= 0
                if side == 0:
                    if other > 0:
                        nxt.append((lw, lo_side))
                    elif lo_side:
                        Z[lw] = k + 1
            pairs = []
            for lv, lof in S:
                c = 2 * k + (1 if (lof or Z[lv] <= k) else 0)
                C[v0 + lv] = c
                pairs.append((v0 + lv, c))
                for u in ci[ro[lv]:ro[lv + 1]]:
                    if v0 <= u < v1:
                        dec(p[v0 + lv], int(u) - v0)
            gathered = [None] * world
            dist.all_gather_object(gathered, pairs)
            assert sum(len(x) for x in gathered) > 0, "stall"
            for r, prs in enumerate(gathered):
                if r == rank:
                    continue
                for v, c in prs:
                    C[v] = c
                    for lw in ghost.get(v, ()):
                        dec(p[v], lw)
            remaining -= sum(len(x) for x in gathered)
            S = nxt
            k += 1
        ref, R, _ = O.color_maxmin(g, seed, with_stats=True)
        q.put((rank, bool((C == ref).all()), k == R))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("scale,seed", [(9, 3), (10, 5)])
def test_partitioned_count_protocol_world2(scale, seed):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_count_protocol_worker, args=(r, 2, port, q, scale, seed))
             for r in range(2)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=300) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    assert all(r[1] for r in res), "replicated colours differ from the oracle"
    assert all(r[2] for r in res), "round count differs from the oracle"


# model of the DEVICE-DRIVEN rounds' exchange (gc_dist_count.cu
# k_dc_persistent), world size 2 on the CPU: every rank pushes
# its coloured pairs into the other rank's inbox (shared memory standing in
# for NVLink peer memory), then writes its mailbox word (epoch | round tag |
# count) there, and polls its own mailbox for the other rank's word.  Inbox
# and mailbox slots alternate with the round's parity; two colourings run
# back to back without clearing anything (the epoch in the word separates
# them); random delays make the ranks drift apart.  Checked against the
# oracle: the colouring, and that both ranks took the same decisions.
def _mailbox_worker(rank, world, port, q, recv, mbox, scale, seeds):
    import random
    import time

    import numpy as np

    import oracle as O
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    rng = random.Random(rank * 7 + 1)
    cap = recv.shape[-1]
    out = []
    try:
        g = G.rmat(scale, 8, seed=3)
        n = g.n
        v0, v1 = gdist.split_range(n, world, rank)
        ro, ci = (t.numpy() for t in gdist.local_rows(g, v0, v1))
        dist.barrier()  # the inboxes exist on every rank (the IPC handle exchange)
        for epoch, seed in enumerate(seeds, start=1):
            p = O.priorities(seed, 0, n).astype(np.int64)
            nl = v1 - v0
            hi = np.zeros(nl, dtype=np.int64)
            lo = np.zeros(nl, dtype=np.int64)
            ghost = {}
            for lv in range(nl):
                row = ci[ro[lv]:ro[lv + 1]].astype(np.int64)
                hi[lv] = int((p[row] > p[v0 + lv]).sum())
                lo[lv] = len(row) - hi[lv]
                for u in row:
                    if not v0 <= u < v1:
                        ghost.setdefault(int(u), []).append(lv)
            UNC, NEVER = 0xFFFFFFFF, 1 << 62
            C = np.full(n, UNC, dtype=np.uint32)
            Z = np.full(nl, NEVER, dtype=np.int64)
            S = [(lv, lo[lv] == 0) for lv in range(nl) if hi[lv] == 0 or lo[lv] == 0]
            k, remaining, totals = 0, n, []
            while remaining > 0:
                par = k & 1
                nxt = []

                def dec(pv, lw):
                    if pv > p[v0 + lw]:
                        hi[lw] -= 1
                        side, other, lo_side = hi[lw], lo[lw], False
                    else:
                        lo[lw] -= 1
                        side, other, lo_side = lo[lw], hi[lw], True
                    assert side >= 0
                    if side == 0:
                        if other > 0:
                            nxt.append((lw, lo_side))
                        elif lo_side:
                            Z[lw] = k + 1
                # A: colour the scheduled vertices, push the pairs into the peer's inbox
                npush = 0
                for lv, lof in S:
                    c = 2 * k + (1 if (lof or Z[lv] <= k) else 0)
                    C[v0 + lv] = c
                    for qq in range(world):
                        if qq != rank:
                            recv[qq, par, rank, npush] = ((v0 + lv) << 32) | c
                    npush += 1
                    for u in ci[ro[lv]:ro[lv + 1]]:
                        if v0 <= u < v1:
                            dec(p[v0 + lv], int(u) - v0)
                assert npush <= cap
                if rng.random() < 0.5:
                    time.sleep(rng.random() * 0.002)
                # B: the mailbox words (after the pairs)
                word = (epoch << 48) | (((k + 1) & 0xFFFF) << 32) | npush
                for qq in range(world):
                    if qq != rank:
                        mbox[qq, par, rank] = word
                # C: wait for every other rank's word of this round and epoch
                tot = npush
                got = {}
                for qq in range(world):
                    if qq == rank:
                        continue
                    t0 = time.time()
                    while (int(mbox[rank, par, qq]) >> 32) != ((epoch << 16) | ((k + 1) & 0xFFFF)):
                        assert time.time() - t0 < 60, "mailbox wait timed out"
                    got[qq] = int(mbox[rank, par, qq]) & 0x3FFFFFFF
                    tot += got[qq]
                assert tot > 0, "stall"
                # D: the received pairs -> colours and ghost rows
                for qq, cnt in got.items():
                    for i in range(cnt):
                        x = int(recv[rank, par, qq, i])
                        v, c = x >> 32, x & 0xFFFFFFFF
                        C[v] = c
                        for lw in ghost.get(v, ()):
                            dec(p[v], lw)
                totals.append(tot)
                remaining -= tot
                S = nxt
                k += 1
            ref, R, _ = O.color_maxmin(g, seed, with_stats=True)
            out.append((bool((C == ref).all()), k == R, totals))
        q.put((rank, out))
    finally:
        dist.destroy_process_group()


def test_device_driven_mailbox_protocol_world2():
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    world, scale = 2, 9
    cap = (1 << scale) // world + 1
    recv = torch.zeros((world, 2, world, cap), dtype=torch.int64).share_memory_()
    mbox = torch.zeros((world, 2, world), dtype=torch.int64).share_memory_()
    procs = [ctx.Process(target=_mailbox_worker, args=(r, world, port, q, recv, mbox, scale, (3, 11)))
             for r in range(world)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=300) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    for run in range(2):
        assert all(r[1][run][0] for r in res), "colouring differs from the oracle"
        assert all(r[1][run][1] for r in res), "round count differs"
        assert res[0][1][run][2] == res[1][1][run][2], "the ranks saw different round totals"
