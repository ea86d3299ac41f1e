"""Parity of the CUDA path (libgc through its C ABI) with the CPU oracle.

Bit-exact comparison of colourings (integer work): every test feeds the same
seeded graph to oracle/ and to libgc and compares element by element.  At the
bench's full size (R-MAT scale 24) the oracle's O(H*m) local certificate --
which determines the colouring uniquely (pinned in test_oracle.py) -- checks
every vertex, alongside the frontier-size trace of a smaller R-MAT.
"""
from __future__ import annotations

import os
import random

import numpy as np
import pytest
import torch

import graphgen as G
import oracle as O
import paper_conf_ipps_osamatybo19_b200 as gcb
from paper_conf_ipps_osamatybo19_b200 import build as gbuild

pytestmark = pytest.mark.gpu

MODES = [gcb.MODE_SWEEP, gcb.MODE_EVENT, gcb.MODE_EVENT_MULTI, gcb.MODE_COUNT]


@pytest.fixture(scope="module", autouse=True)
def _built():
    gbuild.build()
    gcb.lib()


def variant_of(name: str, H: int = 1) -> int:
    if name.startswith("hash_is"):
        return gcb.HASH_IS(int(name[len("hash_is"):]))
    return {"maxmin": gcb.MAXMIN, "luby": gcb.LUBY_MIS, "is_alg2": gcb.IS_ALG2,
            "jp_alg4": gcb.JP_ALG4}.get(name, gcb.MULTIHASH(H))


def oracle_colors(g, seed, variant, H=1):
    if variant.startswith("hash_is"):
        return O.color_hash_is(g, seed, int(variant[len("hash_is"):]))
    if variant == "luby":
        return O.color_luby(g, seed)
    if variant == "is_alg2":
        return O.color_is_alg2(g, seed)
    if variant == "jp_alg4":
        return O.color_jp_alg4(g, seed)
    return O.color_maxmin(g, seed, H)


def gpu_colors(g, seed, vcode, device_out=False, **kw):
    with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
        out = torch.empty(g.n, dtype=torch.int32, device="cuda" if device_out else "cpu")
        out, k, st = h.color(seed, vcode, out, stats=True, **kw)
        return out.cpu().numpy().view(np.uint32), k, st


def supported_modes(vname, H):
    if vname.startswith("hash_is"):
        return [gcb.MODE_AUTO]  # its own per-round kernels; the mode is ignored
    if vname in ("is_alg2", "jp_alg4"):
        return [gcb.MODE_COUNT]
    return [gcb.MODE_SWEEP, gcb.MODE_COUNT] if vname == "luby" else MODES


def jp_depth(g, seed):
    """Longest decreasing-weight path (in vertices): the number of wavefronts
    of the COUNT-mode Luby colouring (test-side definition)."""
    p = O.priorities(seed, 0, g.n).astype(np.int64)
    ro, ci = g.row_offsets.numpy(), g.col_indices.numpy().astype(np.int64)
    depth = np.zeros(g.n, dtype=np.int64)
    for v in np.argsort(-p, kind="stable"):
        nb = ci[ro[v]:ro[v + 1]]
        pred = nb[p[nb] > p[v]]
        depth[v] = 1 + (depth[pred].max() if len(pred) else 0)
    return int(depth.max()) if g.n else 0


# ------------------------------------------------------------- a0 weights
def test_priorities_bit_exact():
    for seed in (1, 42, 2**33 + 5):
        for j in (0, 1, 7, 15):
            for v0, cnt in ((0, 1000), (2**31 - 500, 1000), (2**32 - 300, 300)):
                ref = np.array([O.priority(seed, j, (v0 + i) & 0xFFFFFFFF) for i in range(cnt)],
                               dtype=np.uint32)
                host = torch.empty(cnt, dtype=torch.int32)
                gcb.priorities(seed, j, v0, cnt, host)
                dev = torch.empty(cnt, dtype=torch.int32, device="cuda")
                gcb.priorities(seed, j, v0, cnt, dev)
                assert (host.numpy().view(np.uint32) == ref).all()
                assert (dev.cpu().numpy().view(np.uint32) == ref).all()
    big = torch.empty(1 << 24, dtype=torch.int32, device="cuda")
    gcb.priorities(3, 2, 0, 1 << 24, big)
    assert (big.cpu().numpy().view(np.uint32) == O.priorities(3, 2, 1 << 24)).all()


# ------------------------------------------------------ golden and random
def test_golden_tiny():
    from test_oracle import load_golden
    for name, n, edges, variant, expect in load_golden():
        g = G.csr_from_lists(n, edges)
        H = int(variant[len("multihash"):]) if variant.startswith("multihash") else 1
        vname = "multihash" if variant.startswith("multihash") else variant
        for mode in supported_modes(vname, H):
            C, k, _ = gpu_colors(g, 1, variant_of(vname, H), mode=mode)
            assert C.tolist() == expect, (name, mode)
            assert k == len(set(expect))


@pytest.mark.parametrize("vname,H", [("maxmin", 1), ("multihash", 2), ("multihash", 3),
                                     ("multihash", 16), ("luby", 1), ("is_alg2", 1),
                                     ("jp_alg4", 1)])
def test_random_small_graphs(vname, H):
    rng = random.Random(H * 7 + len(vname))
    for i in range(120):
        n = rng.randint(0, 300)
        p = rng.choice([0.0, 0.01, 0.05, 0.2, 0.5])
        g = G.random_graph(n, p, seed=1000 * H + i)
        seed = rng.getrandbits(64)
        ref = oracle_colors(g, seed, vname, H)
        for mode in supported_modes(vname, H):
            C, k, st = gpu_colors(g, seed, variant_of(vname, H), mode=mode,
                                  thread_deg_max=rng.choice([0, 1, 4, 64]),
                                  hub_deg_min=rng.choice([0, 2, 40, 1 << 20]),
                                  batch_rounds=rng.choice([0, 1, 3]))
            assert (C == ref).all(), (i, n, p, mode)
            assert k == (O.count_colors(ref) if n else 0)


# ------------------------------------------- Hash IS, Alg.6
@pytest.mark.parametrize("T", [0, 1, 4, 16, 64])
def test_hash_is_random_small_graphs(T):
    rng = random.Random(31 + T)
    for i in range(80):
        n = rng.randint(0, 400)
        p = rng.choice([0.0, 0.01, 0.05, 0.2, 0.6])
        g = G.random_graph(n, p, seed=7000 + 100 * T + i)
        seed = rng.getrandbits(64)
        ref, ncol, rounds = O.color_hash_is(g, seed, T, with_stats=True) if n else (
            np.zeros(0, np.uint32), 0, 0)
        C, k, st = gpu_colors(g, seed, gcb.HASH_IS(T))
        assert (C == ref).all(), (i, n, p, T)
        assert k == ncol and st.rounds == rounds


@pytest.mark.parametrize("T", [0, 8])
def test_hash_is_workload_graphs(T):
    # several tiles and ragged tails: R-MAT (hubs, isolated vertices), ER, mesh, rgg
    for g in (G.rmat(14, 16, seed=2), G.erdos_renyi(1 << 15, 8 << 15, seed=2), G.mesh3d(33, 31, 29),
              G.rgg(13, seed=2)):
        ref, ncol, rounds = O.color_hash_is(g, 1, T, with_stats=True)
        C, k, st = gpu_colors(g, 1, gcb.HASH_IS(T), device_out=True)
        assert (C == ref).all(), (g.name, T)
        assert k == ncol and st.rounds == rounds
        assert O.check_proper(g, C) == 0


def test_hash_is_edge_cases():
    cases = [G.csr_from_lists(1, []), G.csr_from_lists(33, []),
             _csr_tensors(20001, [(0, i) for i in range(1, 20001)]),        # hub star
             G.csr_from_lists(700, [(a, b) for a in range(700) for b in range(a + 1, 700)])]  # CTA rows
    for g in cases:
        for T in (0, 2, 64):
            ref = O.color_hash_is(g, 11, T)
            C, k, _ = gpu_colors(g, 11, gcb.HASH_IS(T))
            assert (C == ref).all(), (g.name, T)
    with gcb.Graph(4, torch.tensor([0, 1, 2, 3, 3]), torch.tensor([1, 0, 3], dtype=torch.int32)) as h:
        with pytest.raises(gcb.GCError):
            h.color(1, gcb.HASH_IS(65), torch.empty(4, dtype=torch.int32))


# --------------------------------------------------------------- edge cases
def _csr_tensors(n, pairs):
    return G.csr_from_pairs(n, torch.tensor([a for a, _ in pairs], dtype=torch.int64),
                            torch.tensor([b for _, b in pairs], dtype=torch.int64))


@pytest.mark.parametrize("mode", MODES)
def test_adversarial_shapes(mode):
    cases = [
        G.csr_from_lists(0, []),
        G.csr_from_lists(1, []),
        G.csr_from_lists(33, []),                                 # isolated, n % 32 != 0
        _csr_tensors(200001, [(0, i) for i in range(1, 200001)]),  # hub star K_{1,200000}
        G.csr_from_lists(700, [(a, b) for a in range(700) for b in range(a + 1, 700)]),  # clique
        _csr_tensors(100000, [(i, i + 1) for i in range(99999)]),  # long path
        G.mesh3d(9, 7, 5),
    ]
    for g in cases:
        for vname, H in (("maxmin", 1), ("multihash", 4), ("luby", 1), ("is_alg2", 1),
                         ("jp_alg4", 1)):
            if vname == "luby" and mode not in (gcb.MODE_SWEEP, gcb.MODE_COUNT):
                continue
            if vname in ("is_alg2", "jp_alg4") and mode != gcb.MODE_COUNT:
                continue
            ref = oracle_colors(g, 11, vname, H)
            C, k, st = gpu_colors(g, 11, variant_of(vname, H), mode=mode)
            assert (C == ref).all(), (g.name, vname, H)
            if mode == gcb.MODE_COUNT:  # symmetric input: no fallback out of COUNT mode
                assert st.mode_used == gcb.MODE_COUNT, (g.name, vname)
    # the clique needs exactly n/2 rounds
    g = cases[4]
    _, k, st = gpu_colors(g, 5, gcb.MAXMIN, mode=mode)
    assert st.rounds == 350 and k == 700


def test_duplicates_and_unsorted_rows():
    g = G.erdos_renyi(5000, 40000, seed=3)
    ref = O.color_maxmin(g, 9)
    # shuffle each row and duplicate some entries: adjacency sets are unchanged
    ro, ci = g.row_offsets.tolist(), g.col_indices.tolist()
    rng = random.Random(0)
    rows = []
    for v in range(g.n):
        r = ci[ro[v]:ro[v + 1]]
        r = r + rng.sample(r, min(len(r), 2))
        rng.shuffle(r)
        rows.append(r)
    nro = [0]
    for r in rows:
        nro.append(nro[-1] + len(r))
    g2 = G.Graph(g.n, torch.tensor(nro, dtype=torch.int64),
                 torch.tensor([x for r in rows for x in r], dtype=torch.int32))
    for mode in MODES:
        C, _, st = gpu_colors(g2, 9, gcb.MAXMIN, mode=mode)
        assert (C == ref).all()
        if mode == gcb.MODE_COUNT:  # one-sided duplicates: the deduplicated copy, still COUNT
            assert st.mode_used == gcb.MODE_COUNT
    for vname in ("luby", "is_alg2", "jp_alg4"):
        C, _, st = gpu_colors(g2, 9, variant_of(vname))
        assert (C == oracle_colors(g, 9, vname)).all(), vname
        assert st.mode_used == gcb.MODE_COUNT
    C, _, _ = gpu_colors(g2, 9, gcb.HASH_IS(3))
    assert (C == O.color_hash_is(g, 9, 3)).all()
    C, _, st = gpu_colors(g2, 9, gcb.MULTIHASH(3), mode=gcb.MODE_COUNT)
    assert (C == O.color_maxmin(g, 9, 3)).all() and st.mode_used == gcb.MODE_COUNT
    # the partitioned COUNT rounds deduplicate each partition's rows first
    # (one-sided duplicates would break the count multiset): same colouring
    # at every P, in COUNT mode
    for parts in (1, 2, 4):
        with gcb.loopback_graph(g2.n, g2.row_offsets, g2.col_indices, parts) as h:
            out = torch.empty(g2.n, dtype=torch.int32)
            _, _, st = h.color(9, gcb.MAXMIN, out, stats=True)
            assert st.mode_used == gcb.MODE_COUNT
            assert (out.numpy().view(np.uint32) == ref).all(), parts


def test_dedup_in_row_batches(monkeypatch):
    """The deduplicated copy is built in row batches of < 2^30 entries (CUB's
    int sizes; cfg5 has nnz > 2^31): a tiny batch size (test hook) forces many
    batches, rows longer than a batch included; same colourings."""
    monkeypatch.setenv("GC_DEDUP_BATCH", "700")
    rng = random.Random(4)
    g = G.rmat(12, 16, seed=8)
    ref = O.color_maxmin(g, 2)
    ro, ci = g.row_offsets.tolist(), g.col_indices.tolist()
    rows = []
    for v in range(g.n):
        r = ci[ro[v]:ro[v + 1]]
        r = r + rng.sample(r, min(len(r), 3))
        rng.shuffle(r)
        rows.append(r)
    nro = [0]
    for r in rows:
        nro.append(nro[-1] + len(r))
    assert max(len(r) for r in rows) > 700
    g2 = G.Graph(g.n, torch.tensor(nro, dtype=torch.int64),
                 torch.tensor([x for r in rows for x in r], dtype=torch.int32))
    C, _, st = gpu_colors(g2, 2, gcb.MAXMIN, mode=gcb.MODE_COUNT)
    assert (C == ref).all() and st.mode_used == gcb.MODE_COUNT
    C, _, st = gpu_colors(g2, 2, gcb.LUBY_MIS)
    assert (C == O.color_luby(g, 2)).all() and st.mode_used == gcb.MODE_COUNT


def test_schedule_invariance_and_device_output():
    g = G.rmat(14, 16, seed=2)
    ref = O.color_maxmin(g, 1)
    for mode in MODES:
        for tdm, hub, b in ((1, 2, 1), (8, 4096, 0), (32, 64, 7), (1 << 20, 1 << 30, 2)):
            C, _, _ = gpu_colors(g, 1, gcb.MAXMIN, mode=mode, thread_deg_max=tdm,
                                 hub_deg_min=hub, batch_rounds=b, device_out=True)
            assert (C == ref).all()


def test_errors():
    ro = torch.tensor([0, 1, 2], dtype=torch.int64)
    with pytest.raises(gcb.GCError) as e:
        gcb.Graph(2, ro, torch.tensor([0, 0], dtype=torch.int32))      # self-loop
    assert e.value.code == -2
    with pytest.raises(gcb.GCError) as e:
        gcb.Graph(2, ro, torch.tensor([5, 0], dtype=torch.int32))      # col >= n
    assert e.value.code == -1
    with pytest.raises(gcb.GCError) as e:
        gcb.Graph(3, torch.tensor([0, 1, 1, 1]), torch.tensor([1], dtype=torch.int32),
                  flags=gcb.VALIDATE)                                   # not symmetric
    assert e.value.code == -3
    # an asymmetric adjacency SET (0 -> 1 only), not validated at create: the
    # COUNT kernels detect it (underflow / stall) and report it, never a
    # silently wrong colouring; Alg.4 has no fallback kernel
    asym = gcb.Graph(3, torch.tensor([0, 1, 1, 1]), torch.tensor([1], dtype=torch.int32))
    with pytest.raises(gcb.GCError) as e:
        asym.color(1, gcb.JP_ALG4)
    assert e.value.code == -3
    asym.close()
    g = gcb.Graph(2, ro, torch.tensor([1, 0], dtype=torch.int32))
    with pytest.raises(gcb.GCError):
        g.color(1, gcb.MULTIHASH(17))
    with pytest.raises(gcb.GCError):
        g.color(1, 99)
    g.close()


def test_compact_and_count_colors():
    g = G.erdos_renyi(20000, 160000, seed=5)
    raw = O.color_maxmin(g, 2)
    C, k, _ = gpu_colors(g, 2, gcb.MAXMIN, flags=gcb.COMPACT)
    assert (C == O.compact_colors(raw)).all()
    assert k == O.count_colors(raw) == int(C.max()) + 1
    assert gcb.count_colors(torch.from_numpy(raw.view(np.int32))) == k
    assert gcb.count_colors(torch.from_numpy(raw.view(np.int32)).cuda()) == k


def test_borrow_device_and_stream():
    g = G.rmat(12, 16, seed=4).to("cuda")
    ref = O.color_maxmin(g.to("cpu"), 3)
    s = torch.cuda.Stream()
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        h.set_stream(s)
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        with torch.cuda.stream(s):
            h.color(3, gcb.MAXMIN, out)
        s.synchronize()
        assert (out.cpu().numpy().view(np.uint32) == ref).all()


def test_memory_cache_reuse_and_trim():
    """Handles of different sizes reuse the library's cached blocks (gc_alloc.cu):
    stale contents of a reused block must never leak into a later colouring."""
    graphs = [G.rmat(s, 8, seed=s) for s in (13, 11, 13, 12)]
    refs = [O.color_maxmin(g, 5) for g in graphs]
    for rep in range(2):
        for g, ref in zip(graphs, refs):
            for mode in (gcb.MODE_EVENT, gcb.MODE_SWEEP):
                got, _, _ = gpu_colors(g, 5, gcb.MAXMIN, mode=mode)
                assert (got == ref).all()
        gcb.trim()


# ----------------------------------------------------------- config sizes
@pytest.mark.parametrize("mode", MODES)
def test_cfg1_grid(mode):
    g = G.config_graph("cfg1")
    ref, R, nk = O.color_maxmin(g, 1, with_stats=True)
    C, k, st = gpu_colors(g, 1, gcb.MAXMIN, mode=mode, frontier_cap=64)
    assert (C == ref).all() and st.rounds == R and st.frontier_sizes == nk


def test_cfg2_er_luby_and_maxmin():
    g = G.config_graph("cfg2", device="cuda").to("cpu")
    ref, ncol, inner = O.color_luby(g, 1, with_stats=True)
    C, k, st = gpu_colors(g, 1, gcb.LUBY_MIS, mode=gcb.MODE_SWEEP)
    assert (C == ref).all() and k == ncol and st.inner_iterations == inner
    C, k, st = gpu_colors(g, 1, gcb.LUBY_MIS)  # AUTO: COUNT (wavefronts)
    assert st.mode_used == gcb.MODE_COUNT
    assert (C == ref).all() and k == ncol and st.rounds == jp_depth(g, 1)
    ref2, R, nk = O.color_maxmin(g, 1, with_stats=True)
    for mode in MODES:
        C, k, st = gpu_colors(g, 1, gcb.MAXMIN, mode=mode, frontier_cap=4096)
        assert (C == ref2).all() and st.rounds == R and st.frontier_sizes == nk


@pytest.mark.parametrize("H", [1, 2, 4, 8])
def test_cfg3_mesh_multihash(H):
    g = G.config_graph("cfg3", device="cuda").to("cpu")
    ref, R, nk = O.color_maxmin(g, 1, H, with_stats=True)
    for mode in MODES:
        C, k, st = gpu_colors(g, 1, gcb.MULTIHASH(H), mode=mode, frontier_cap=4096)
        assert (C == ref).all() and st.rounds == R and st.frontier_sizes == nk


def test_rmat_s18_full_oracle():
    g = G.rmat(18, 16, seed=1, device="cuda").to("cpu")
    ref, R, nk = O.color_maxmin(g, 1, with_stats=True)
    for mode in MODES:
        C, k, st = gpu_colors(g, 1, gcb.MAXMIN, mode=mode, frontier_cap=8192)
        assert (C == ref).all() and st.rounds == R and st.frontier_sizes == nk
    ref_l = O.color_luby(g, 1)
    for mode in (gcb.MODE_SWEEP, gcb.MODE_COUNT):
        C, k, st = gpu_colors(g, 1, gcb.LUBY_MIS, mode=mode)
        assert (C == ref_l).all()
    C, k, st = gpu_colors(g, 1, gcb.MULTIHASH(4))
    assert (C == O.color_maxmin(g, 1, 4)).all()


def test_cfg4_rmat_s24_certificate():
    """Full bench size, bench launch configuration (defaults): the certificate
    (unique characterisation of the max-min colouring) checks every vertex,
    plus properness and the 2R identity."""
    g = G.config_graph("cfg4", device="cuda")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, k, st = h.color(1, gcb.MAXMIN, out, stats=True)
    C = out.cpu().numpy().view(np.uint32)
    gh = g.to("cpu")
    assert O.cert_maxmin(gh, 1, 1, C) == 0
    assert O.check_proper(gh, C) == 0
    assert k == O.count_colors(C) and k in (2 * st.rounds - 1, 2 * st.rounds)


def test_cfg4_rmat_s24_multihash_certificate():
    """Multi-hash H=4 (COUNT mode under AUTO) at the bench size: the O(H*m)
    certificate checks every vertex."""
    g = G.config_graph("cfg4", device="cuda")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, k, st = h.color(1, gcb.MULTIHASH(4), out, stats=True)
    assert st.mode_used == gcb.MODE_COUNT
    C = out.cpu().numpy().view(np.uint32)
    gh = g.to("cpu")
    assert O.cert_maxmin(gh, 1, 4, C) == 0
    assert O.check_proper(gh, C) == 0


def test_luby_count_wavefronts_and_wide_mex():
    """COUNT-mode Luby: wavefront count = longest decreasing-weight path on
    random graphs; cliques whose mex passes the 1024-colour slot window (the
    rescan path) and a hub star; asymmetric input falls back to SWEEP."""
    rng = random.Random(5)
    for i in range(40):
        g = G.random_graph(rng.randint(1, 400), rng.choice([0.01, 0.05, 0.3]), seed=77 + i)
        C, k, st = gpu_colors(g, i, gcb.LUBY_MIS, mode=gcb.MODE_COUNT)
        assert (C == O.color_luby(g, i)).all() and st.rounds == jp_depth(g, i)
    for n in (33, 1023, 1030, 2200):
        g = G.csr_from_lists(n, [(a, b) for a in range(n) for b in range(a + 1, n)])
        C, k, st = gpu_colors(g, 3, gcb.LUBY_MIS, mode=gcb.MODE_COUNT)
        # closed form of the Luby colouring (pinned equal in test_oracle.py)
        assert (C == O.color_greedy_by_priority(g, 3)).all() and k == n and st.rounds == n
    g = _csr_tensors(300001, [(0, i) for i in range(1, 300001)] + [(1, 2), (2, 3)])
    C, k, st = gpu_colors(g, 2, gcb.LUBY_MIS, mode=gcb.MODE_COUNT)
    assert (C == O.color_luby(g, 2)).all()


def test_cfg4_rmat_s24_luby_certificate():
    """Luby-MIS (COUNT mode) at the bench size: the mex certificate
    (first-fit in decreasing weight order, characterises it uniquely)."""
    g = G.config_graph("cfg4", device="cuda")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, k, st = h.color(1, gcb.LUBY_MIS, out, stats=True)
    assert st.mode_used == gcb.MODE_COUNT
    C = out.cpu().numpy().view(np.uint32)
    gh = g.to("cpu")
    assert O.cert_mex(gh, 1, C) == 0
    assert O.check_proper(gh, C) == 0
    assert k == O.count_colors(C) == int(C.max()) + 1


# ------------------------------------------------- partitioned (row e)
@pytest.mark.parametrize("parts", [1, 2, 3, 4, 8])
def test_loopback_partitions(parts):
    """The multi-GPU algorithm (per-partition replicas + per-round exchange of
    coloured pairs) with `parts` partitions on one GPU equals the oracle."""
    for g, vname, H in ((G.rmat(14, 16, seed=5), "maxmin", 1),
                        (G.erdos_renyi(50000, 400000, seed=6), "maxmin", 1),
                        (G.rmat(13, 16, seed=7), "multihash", 3),
                        (G.csr_from_lists(5, [(0, 1), (1, 2)]), "maxmin", 1)):
        ref, R, nk = O.color_maxmin(g, 9, H, with_stats=True)
        modes = [gcb.MODE_AUTO, gcb.MODE_SWEEP] if H == 1 else [gcb.MODE_AUTO]
        with gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, parts) as h:
            for mode in modes:
                out = torch.empty(g.n, dtype=torch.int32)
                _, k, st = h.color(9, variant_of(vname, H), out, stats=True, frontier_cap=8192,
                                   mode=mode)
                assert st.mode_used == (gcb.MODE_COUNT if H == 1 and mode == gcb.MODE_AUTO
                                        else gcb.MODE_SWEEP)
                assert (out.numpy().view(np.uint32) == ref).all(), (parts, g.name, mode)
                assert st.rounds == R and st.frontier_sizes == nk and k == O.count_colors(ref)
            outc = torch.empty(g.n, dtype=torch.int32)
            h.color(9, variant_of(vname, H), outc, flags=gcb.COMPACT)
            assert (outc.numpy().view(np.uint32) == O.compact_colors(ref)).all()


@pytest.mark.parametrize("parts", [2, 8])
def test_loopback_count_hubs_and_ghost_rows(parts):
    """Distributed COUNT rounds on skewed graphs: hub rows longer than the
    block-chunk threshold (own and ghost rows), a star across partitions."""
    cases = [G.rmat(16, 16, seed=3),
             _csr_tensors(20001, [(0, i) for i in range(1, 20001)] + [(5, 9), (9, 17)])]
    for g in cases:
        ref, R, nk = O.color_maxmin(g, 4, with_stats=True)
        with gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, parts) as h:
            out = torch.empty(g.n, dtype=torch.int32)
            _, k, st = h.color(4, gcb.MAXMIN, out, stats=True, frontier_cap=1 << 16)
            assert (out.numpy().view(np.uint32) == ref).all()
            assert st.rounds == R and st.frontier_sizes == nk


@pytest.mark.parametrize("parts", [3, 4, 8])
def test_loopback_repeated_colourings_stable(parts):
    """Device-driven partitioned rounds repeated back to back (a race between
    a fast block freeing round-(k+2) vertices and a slow block reading round
    k+1's scheduled slice once showed up only after several colourings): 24
    colourings of one handle, each equal to the oracle."""
    g = G.rmat(18, 16, seed=11)
    ref = O.color_maxmin(g, 2)
    with gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, parts) as h:
        out = torch.empty(g.n, dtype=torch.int32)
        for i in range(24):
            h.color(2, gcb.MAXMIN, out, mode=gcb.MODE_COUNT)
            assert (out.numpy().view(np.uint32) == ref).all(), (parts, i)


def test_cfg5_style_partitioned_rmat_s25():
    """cfg5's check at the largest size a test affords: R-MAT s25 (1.08e9
    entries) partitioned P = 2, 4 (loopback transport: the same COUNT rounds,
    ghost rows and pair exchange as NCCL) equals P = 1 element by element, and
    the P = 1 colouring passes the oracle's certificate."""
    g = G.rmat(25, 16, seed=1, device="cuda")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        one = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, k1, st1 = h.color(1, gcb.MAXMIN, one, stats=True)
    for parts in (2, 4):
        with gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, parts) as h:
            outp = torch.empty(g.n, dtype=torch.int32, device="cuda")
            _, kp, stp = h.color(1, gcb.MAXMIN, outp, stats=True)
        assert stp.mode_used == gcb.MODE_COUNT
        assert torch.equal(outp, one) and kp == k1 and stp.rounds == st1.rounds, parts
    C = one.cpu().numpy().view(np.uint32)
    gh = g.to("cpu")
    assert O.cert_maxmin(gh, 1, 1, C) == 0


@pytest.mark.parametrize("scale", [16, 20])
def test_rgg_workloads_all_variants(scale):
    """the random geometric graphs of the paper's scaling study
    (rgg_n_2_<scale>, Table I, Fig.3) -- every variant
    element by element against the oracle (rounds too, where defined), in the
    launch configuration AUTO picks."""
    g = G.rgg(scale, seed=1, device="cuda").to("cpu")
    cases = [("maxmin", 1), ("multihash", 4), ("luby", 1), ("is_alg2", 1), ("jp_alg4", 1),
             ("hash_is8", 1)]
    for vname, H in cases:
        C, k, st = gpu_colors(g, 1, variant_of(vname, H), frontier_cap=4096)
        ref = oracle_colors(g, 1, vname, H)
        assert (C == ref).all(), vname
        assert k == O.count_colors(ref), vname
        if vname in ("maxmin", "multihash"):
            _, R, nk = O.color_maxmin(g, 1, H, with_stats=True)
            assert st.rounds == R and st.frontier_sizes == nk
        if vname in ("is_alg2", "jp_alg4"):
            _, R = (O.color_is_alg2 if vname == "is_alg2" else O.color_jp_alg4)(g, 1, with_stats=True)
            assert st.rounds == R


LDF_VARIANTS = [("maxmin", gcb.MAXMIN, lambda g, s: O.color_maxmin(g, s, ldf=True)),
                ("luby", gcb.LUBY_MIS, lambda g, s: O.color_luby(g, s, ldf=True)),
                ("is_alg2", gcb.IS_ALG2, lambda g, s: O.color_is_alg2(g, s, ldf=True)),
                ("jp_alg4", gcb.JP_ALG4, lambda g, s: O.color_jp_alg4(g, s, ldf=True))]


def test_ldf_random_and_workload_graphs():
    """largest-degree-first priorities (R21) in the COUNT kernels,
    element by element against the oracle: random graphs, duplicate entries
    (the degree counts distinct neighbours), a star (closed form), R-MAT s16,
    ER, the mesh and RGG; max-min rounds and frontier sizes too."""
    rng = random.Random(12)
    graphs = [G.random_graph(rng.randint(1, 300), rng.choice([0.02, 0.1, 0.4]), seed=500 + i)
              for i in range(60)]
    graphs += [G.rmat(16, 16, seed=2), G.erdos_renyi(30000, 240000, seed=4), G.mesh3d(24, 24, 24),
               G.rgg(15, seed=1), _csr_tensors(5001, [(0, i) for i in range(1, 5001)])]
    for i, g in enumerate(graphs):
        for name, v, ref_fn in LDF_VARIANTS:
            C, k, st = gpu_colors(g, 1 + i % 5, gcb.LDF(v), frontier_cap=8192)
            ref = ref_fn(g, 1 + i % 5)
            assert st.mode_used == gcb.MODE_COUNT
            assert (C == ref).all(), (name, g.name, i)
            if name == "maxmin":
                _, R, nk = O.color_maxmin(g, 1 + i % 5, with_stats=True, ldf=True)
                assert st.rounds == R and st.frontier_sizes == nk
    star = graphs[-1]
    C, _, _ = gpu_colors(star, 3, gcb.LDF(gcb.MAXMIN))
    assert C[0] == 0 and (C[1:] == 1).all()
    # duplicates + shuffled rows: same colouring as the clean graph
    g = G.erdos_renyi(4000, 30000, seed=8)
    ro, ci = g.row_offsets.tolist(), g.col_indices.tolist()
    rows = []
    for v in range(g.n):
        r = ci[ro[v]:ro[v + 1]]
        r = r + rng.sample(r, min(len(r), 2))
        rng.shuffle(r)
        rows.append(r)
    nro = [0]
    for r in rows:
        nro.append(nro[-1] + len(r))
    g2 = G.Graph(g.n, torch.tensor(nro, dtype=torch.int64),
                 torch.tensor([x for r in rows for x in r], dtype=torch.int32))
    for name, v, ref_fn in LDF_VARIANTS:
        C, _, _ = gpu_colors(g2, 5, gcb.LDF(v))
        assert (C == ref_fn(g, 5)).all(), name


def test_ldf_rmat_s24_certificates_and_errors():
    """LDF at the bench size: the max-min certificate and the mex certificate
    with (degree, weight) keys check every vertex; LDF with multi-hash, Hash IS
    or a partitioned handle is rejected."""
    g = G.config_graph("cfg4", device="cuda")
    gh = g.to("cpu")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, k, st = h.color(1, gcb.LDF(gcb.MAXMIN), out, stats=True)
        C = out.cpu().numpy().view(np.uint32)
        assert O.cert_maxmin(gh, 1, 1, C, ldf=True) == 0 and O.check_proper(gh, C) == 0
        assert k in (2 * st.rounds - 1, 2 * st.rounds)
        _, k, st = h.color(1, gcb.LDF(gcb.LUBY_MIS), out, stats=True)
        L = out.cpu().numpy().view(np.uint32)
        assert O.cert_mex(gh, 1, L, ldf=True) == 0 and O.check_proper(gh, L) == 0
        for bad in (gcb.LDF(gcb.MULTIHASH(2)), gcb.LDF(gcb.HASH_IS(4)), gcb.MAXMIN | (1 << 20)):
            with pytest.raises(gcb.GCError) as e:
                h.color(1, bad, out)
            assert e.value.code == -1


def test_cfg5_rmat_s27_one_gpu_and_partitions():
    """cfg5 at its stated size: R-MAT s27 ef16 (1.3e8 vertices, nnz > 2^31).
    One B200 colours it through gc_create_csr / AUTO (the bench launch
    configuration); the partitioned algorithm (loopback transport: the same
    COUNT rounds, ghost rows and pair exchange as over NCCL) at P = 2, 4, 8
    equals P = 1 bit for bit; on the host the oracle's O(m)
    certificate -- which determines the max-min colouring uniquely (App. C
    #4, mutation-pinned in test_oracle.py) -- checks every vertex, plus
    properness and n_colors in {2R-1, 2R}."""
    g = G.rmat(27, 16, seed=1, device="cuda", pieces=8)
    assert g.n == 1 << 27 and g.nnz > 2 ** 31
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        one = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, k1, st1 = h.color(1, gcb.MAXMIN, one, stats=True)
    assert st1.mode_used == gcb.MODE_COUNT
    for parts in (2, 4, 8):
        with gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, parts) as h:
            outp = torch.empty(g.n, dtype=torch.int32, device="cuda")
            _, kp, stp = h.color(1, gcb.MAXMIN, outp, stats=True)
        assert stp.mode_used == gcb.MODE_COUNT
        assert torch.equal(outp, one) and kp == k1 and stp.rounds == st1.rounds, parts
        del outp
        gcb.trim()
    C = one.cpu().numpy().view(np.uint32)
    gh = g.to("cpu")
    del g, one
    torch.cuda.empty_cache()
    assert O.cert_maxmin(gh, 1, 1, C) == 0
    assert O.check_proper(gh, C) == 0
    assert k1 == O.count_colors(C) and k1 in (2 * st1.rounds - 1, 2 * st1.rounds)


@pytest.mark.skipif(os.environ.get("GC_SLOW_TESTS") != "1",
                    reason="about 10 min of oracle time on the host: GC_SLOW_TESTS=1")
def test_cfg4_rmat_s24_full_oracle_elementwise():
    """The bench graph (R-MAT s24) against the full oracle colouring (Alg.1 +
    Alg.5 with snapshot rounds, not the certificate), element by element,
    with the round count and the per-round frontier sizes."""
    g = G.config_graph("cfg4", device="cuda")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, k, st = h.color(1, gcb.MAXMIN, out, stats=True, frontier_cap=1 << 14)
    C = out.cpu().numpy().view(np.uint32)
    gh = g.to("cpu")
    del g
    ref, R, nk = O.color_maxmin(gh, 1, with_stats=True)
    assert (C == ref).all()
    assert st.rounds == R and st.frontier_sizes == nk and k == O.count_colors(ref)


@pytest.mark.parametrize("vname", ["is_alg2", "jp_alg4"])
def test_alg2_alg4_scaled(vname):
    """SURVEY N3 at scale: R-MAT s18 and cfg2 ER against the oracle (rounds
    too), a clique (colours = ranks) and a 70k-vertex path (Alg.4)."""
    fn = O.color_is_alg2 if vname == "is_alg2" else O.color_jp_alg4
    for g in (G.rmat(18, 16, seed=1, device="cuda").to("cpu"),
              G.config_graph("cfg2", device="cuda").to("cpu")):
        ref, R = fn(g, 1, with_stats=True)
        C, k, st = gpu_colors(g, 1, variant_of(vname))
        assert st.mode_used == gcb.MODE_COUNT
        assert (C == ref).all() and st.rounds == R and k == O.count_colors(ref)
    if vname == "jp_alg4":
        n = 1200
        g = G.csr_from_lists(n, [(a, b) for a in range(n) for b in range(a + 1, n)])
        C, k, st = gpu_colors(g, 2, gcb.JP_ALG4)
        assert (C == O.color_greedy_by_priority(g, 2)).all() and k == n
        # a long path: tens of thousands of rounds, colours alternate
        g = _csr_tensors(70001, [(i, i + 1) for i in range(70000)])
        C, k, st = gpu_colors(g, 3, gcb.JP_ALG4)
        assert (C == O.color_jp_alg4(g, 3)).all()


def _sparse_hubs_graph(n, hubs, hub_deg, leaf_pairs, seed):
    """Long runs of isolated vertices (more than 32 rows without entries
    inside one 512-entry warp tile), a few hubs whose rows cross many tiles,
    and scattered rows of 1-3 entries: the shapes the counting pass's warp
    tiles walk row chunk by row chunk."""
    rng = random.Random(seed)
    pairs = set()
    for h in hubs:
        for _ in range(hub_deg):
            u = rng.randrange(n)
            if u != h:
                pairs.add((min(h, u), max(h, u)))
    for _ in range(leaf_pairs):
        a, b = rng.randrange(0, n, 97), rng.randrange(n)  # sparse: most rows stay empty
        if a != b:
            pairs.add((min(a, b), max(a, b)))
    return _csr_tensors(n, sorted(pairs))


def test_counting_pass_tiles_and_row_runs():
    """COUNT mode's counting pass (warp tiles over the entries, row chunks of
    32, rows crossing tile boundaries pre-zeroed, rows without entries left to
    the init phase) against the oracle, element by element, for max-min and
    Luby (the same pass with lo pinned), on graphs with long runs of empty
    rows, hubs spanning many tiles and short rows; several seeds on one
    handle (the per-graph tile table is reused); a CSR borrowed at a 4-byte
    offset (not 16-byte aligned: the degree-binned pass) gives the same."""
    graphs = [_sparse_hubs_graph(60000, [5, 30001, 59999], 6000, 4000, 1),
              _sparse_hubs_graph(9000, [0, 4500], 2500, 300, 2),
              G.rmat(14, 4, seed=5)]
    for g in graphs:
        with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
            for seed in (1, 7, 123):
                for vname in ("maxmin", "luby"):
                    out = torch.empty(g.n, dtype=torch.int32)
                    _, _, st = h.color(seed, variant_of(vname), out, stats=True, mode=gcb.MODE_COUNT)
                    assert st.mode_used == gcb.MODE_COUNT
                    assert (out.numpy().view(np.uint32) == oracle_colors(g, seed, vname)).all(), (g.name, seed, vname)
    g = graphs[0]
    ci = torch.empty(g.nnz + 1, dtype=torch.int32, device="cuda")
    ci[1:] = g.col_indices.to("cuda")
    ro = g.row_offsets.to("cuda")
    with gcb.Graph(g.n, ro, ci[1:], flags=gcb.BORROW_DEVICE) as h:
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        _, _, st = h.color(7, gcb.MAXMIN, out, stats=True, mode=gcb.MODE_COUNT)
        assert st.mode_used == gcb.MODE_COUNT
        assert (out.cpu().numpy().view(np.uint32) == O.color_maxmin(g, 7)).all()


_OVERFLOW_CHECK = r"""
import sys
import numpy as np, torch
sys.path.insert(0, sys.argv[1])
import graphgen as G, oracle as O, paper_conf_ipps_osamatybo19_b200 as gcb
def star(n):
    return G.csr_from_pairs(n, torch.zeros(n - 1, dtype=torch.int64), torch.arange(1, n, dtype=torch.int64))
cases = [G.rmat(13, 16, seed=3), G.erdos_renyi(3000, 30000, seed=2), star(20001), G.rmat(16, 16, seed=9)]
refs = {"maxmin": lambda g: O.color_maxmin(g, 5), "luby": lambda g: O.color_luby(g, 5),
        "mh3": lambda g: O.color_maxmin(g, 5, 3), "alg2": lambda g: O.color_is_alg2(g, 5),
        "alg4": lambda g: O.color_jp_alg4(g, 5)}
codes = {"maxmin": gcb.MAXMIN, "luby": gcb.LUBY_MIS, "mh3": gcb.MULTIHASH(3), "alg2": gcb.IS_ALG2,
         "alg4": gcb.JP_ALG4}
for g in cases:
    with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
        for name, code in codes.items():
            out = torch.empty(g.n, dtype=torch.int32)
            _, _, st = h.color(5, code, out, stats=True, mode=gcb.MODE_COUNT)
            assert st.mode_used == gcb.MODE_COUNT, (g.name, name)
            assert (out.numpy().view(np.uint32) == refs[name](g)).all(), (g.name, name)
print("overflow paths ok")
"""


def test_count_overflow_paths(tmp_path):
    """COUNT rounds from a build whose per-block item staging and fresh list
    hold 4 / 8 entries (GC_STAGE_ITEMS=4): freed vertices overflow into direct
    scheduling by the walking warp, staged items spill straight to the global
    lists, long rows that do not fit leave holes -- paths a normal build takes
    only in extreme rounds.  Same colourings as the oracle for max-min, Luby,
    multi-hash, Alg.2 and Alg.4 (a subprocess loads the variant library)."""
    import subprocess
    import sys as _sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    lib = str(tmp_path / "libgc_stage4.so")
    gbuild.build(out=lib, defines=["GC_STAGE_ITEMS=4"])
    env = dict(os.environ, GC_LIB_PATH=lib)
    r = subprocess.run([_sys.executable, "-c", _OVERFLOW_CHECK, root], env=env, capture_output=True, text=True,
                       timeout=900)
    assert r.returncode == 0 and "overflow paths ok" in r.stdout, r.stdout[-2000:] + r.stderr[-4000:]


def test_counting_pass_long_isolated_runs():
    """Millions of isolated vertices between a few edges (one warp tile spans
    them all): the counting pass jumps over runs of empty rows by binary
    search instead of walking them 32 at a time; same colourings as the
    oracle, and an edgeless graph of 2^22 vertices colours fast."""
    import time
    n = 3_000_000
    pairs = [(0, 1), (1, 2), (2, 3), (0, 3), (5, n - 7), (n - 3, n - 2), (n - 2, n - 1), (17, n // 2), (n // 2, n // 2 + 1)]
    g = _csr_tensors(n, pairs)
    for vname in ("maxmin", "luby"):
        C, _, st = gpu_colors(g, 3, variant_of(vname), mode=gcb.MODE_COUNT)
        assert st.mode_used == gcb.MODE_COUNT
        assert (C == oracle_colors(g, 3, vname)).all(), vname
    e = G.csr_from_lists(1 << 22, [])
    with gcb.Graph(e.n, e.row_offsets, e.col_indices) as h:
        out = torch.empty(e.n, dtype=torch.int32)
        h.color(1, gcb.MAXMIN, out, mode=gcb.MODE_COUNT)
        t0 = time.perf_counter()
        _, k, st = h.color(2, gcb.MAXMIN, out, stats=True, mode=gcb.MODE_COUNT)
        dt = time.perf_counter() - t0
    assert k == 1 and st.rounds == 1 and (out.numpy() == 1).all()
    assert dt < 0.5, dt


def test_relaxed_rounds_repeated_colourings():
    """The relaxed rounds (max-min; Luby and Alg.2 through the JP kernel)
    publish items through round tags and read earlier rounds' single-writer
    words until written: many colourings with different seeds on ONE handle
    (item arrays reused across colourings, epoch tags) against the oracle,
    element by element."""
    g = G.rmat(16, 16, seed=21)
    with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
        for seed in range(1, 13):
            for vname in ("maxmin", "luby", "is_alg2"):
                out = torch.empty(g.n, dtype=torch.int32)
                _, _, st = h.color(seed, variant_of(vname), out, stats=True, mode=gcb.MODE_COUNT)
                assert st.mode_used == gcb.MODE_COUNT
                assert (out.numpy().view(np.uint32) == oracle_colors(g, seed, vname)).all(), (seed, vname)
