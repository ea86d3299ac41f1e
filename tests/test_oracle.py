"""Pins of the CPU oracle (oracle/) against things other than itself.

Every check here is independent of the oracle's own arithmetic: published
hash vectors, an inverse derived from number theory, hand-derived golden
colourings, a separate literal (in-place, random thread order) transcription
of the paper's Algorithm 5, closed forms, textbook greedy colourings, a
Jones-Plassmann implementation, local certificates and brute-force chromatic
numbers.  See DESIGN.md "Oracle pins".
"""
from __future__ import annotations

import itertools
import os
import random

import numpy as np
import pytest
import torch

import graphgen as G
import oracle as O

GOLDEN = os.path.join(os.path.dirname(__file__), "golden", "tiny_colorings.txt")
M32 = 0xFFFFFFFF


# ------------------------------------------------------------------ helpers
def adjacency(g):
    ro = g.row_offsets.tolist()
    ci = g.col_indices.tolist()
    return [ci[ro[v]:ro[v + 1]] for v in range(g.n)]


def fmix32_inverse(h: int) -> int:
    """Inverse of MurmurHash3's fmix32 derived independently: xorshift by
    s >= 16 is an involution, by 13 inverts with shifts 13 and 26, and the odd
    multipliers invert modulo 2^32."""
    inv1 = pow(0x85EBCA6B, -1, 1 << 32)
    inv2 = pow(0xC2B2AE35, -1, 1 << 32)
    h ^= h >> 16
    h = (h * inv2) & M32
    h ^= (h >> 13) ^ (h >> 26)
    h = (h * inv1) & M32
    h ^= h >> 16
    return h


def ldf_key(adj, seed):
    """R21 restated with Python tuples: priority of v under hash j is
    (deg(v), p_j(v)), compared lexicographically (largest degree first)."""
    return lambda j, v: (len(adj[v]), O.priority(seed, j, v))


def alg5_literal(n, adj, seed, H, rng, key=None):
    """PAPER.md Algorithm 5 transcribed line by line, 1-based colours, IN PLACE,
    threads in a random order each iteration (the GPU's nondeterministic
    schedule).  Generalised to H hashes by letting hash j of an iteration use
    colour = 2*(iteration*H + j); the L26 test skips u iff C[u] is valid and not
    one of this iteration's colours.  Returns 0-based colours (paper - 1)."""
    INVALID = 0
    key = key or (lambda j, v: O.priority(seed, j, v))
    R = [[key(j, v) for v in range(n)] for j in range(H)]                 # L7
    C = [INVALID] * n                                                      # L5
    iteration = 0                                                          # L3
    while any(c == INVALID for c in C):                                    # L9
        lo_col, hi_col = 2 * iteration * H + 1, 2 * iteration * H + 2 * H
        F = list(range(n))                                                 # L8
        rng.shuffle(F)
        for v in F:                                                        # L16
            if C[v] != INVALID:                                            # L18
                continue
            for j in range(H):
                colormax = True                                            # L21
                colormin = True                                            # L22
                color = 2 * (iteration * H + j)                            # L23
                for u in adj[v]:                                           # L25
                    if C[u] != INVALID and not (lo_col <= C[u] <= hi_col):  # L26
                        continue
                    if R[j][v] <= R[j][u]:                                 # L29
                        colormax = False
                    if R[j][v] >= R[j][u]:                                 # L32
                        colormin = False
                new = INVALID
                if colormax:                                               # L37
                    new = color + 1
                if colormin:                                               # L40
                    new = color + 2
                if new != INVALID:
                    C[v] = new
                    break
        iteration += 1
    return [c - 1 for c in C], iteration


def jones_plassmann(n, adj, seed, key=None):
    """Jones-Plassmann: a vertex colours itself with the smallest
    colour unused by its neighbours once every higher-weight neighbour is
    coloured.  Synchronous rounds."""
    key = key or (lambda j, v: O.priority(seed, j, v))
    p = [key(0, v) for v in range(n)]
    C = [None] * n
    while any(c is None for c in C):
        ready = [v for v in range(n) if C[v] is None and
                 all(C[u] is not None for u in adj[v] if p[u] > p[v])]
        newc = {}
        for v in ready:
            used = {C[u] for u in adj[v] if C[u] is not None}
            c = 0
            while c in used:
                c += 1
            newc[v] = c
        for v, c in newc.items():
            C[v] = c
    return C


def first_fit(n, adj, order):
    """Textbook sequential greedy."""
    C = [None] * n
    for v in order:
        used = {C[u] for u in adj[v] if C[u] is not None}
        c = 0
        while c in used:
            c += 1
        C[v] = c
    return C


def chromatic_number(n, adj):
    """Brute force: smallest k admitting a proper colouring (n <= 9)."""
    if n == 0:
        return 0
    for k in range(1, n + 1):
        C = [-1] * n

        def bt(i):
            if i == n:
                return True
            for c in range(k):
                if all(C[u] != c for u in adj[i]):
                    C[i] = c
                    if bt(i + 1):
                        return True
            C[i] = -1
            return False

        if bt(0):
            return k
    return n


def random_graphs(count, nmax, seed0=0):
    rng = random.Random(seed0)
    for i in range(count):
        n = rng.randint(1, nmax)
        p = rng.choice([0.05, 0.15, 0.3, 0.6, 0.9])
        yield G.random_graph(n, p, seed=seed0 * 100003 + i)


def load_golden():
    rows = []
    for line in open(GOLDEN):
        line = line.strip()
        if not line or line.startswith("#"):
            continue
        name, n, edges, variant, colors = [x.strip() for x in line.split("|")]
        n = int(n)
        el = [tuple(map(int, e.split("-"))) for e in edges.split(",")] if edges else []
        rows.append((name, n, el, variant, [int(c) for c in colors.split()]))
    return rows


# ------------------------------------------------------------------ weights
def test_fmix32_smhasher_vectors():
    # MurmurHash3_x86_32 of the empty key reduces to fmix32(seed); SMHasher's
    # published vectors: seed 0 -> 0, seed 1 -> 0x514E28B7,
    # seed 0xFFFFFFFF -> 0x81F16F39.
    assert O.fmix32(0) == 0
    assert O.fmix32(1) == 0x514E28B7
    assert O.fmix32(0xFFFFFFFF) == 0x81F16F39


def test_weights_bijective_and_distinct():
    rng = random.Random(5)
    for seed in (0, 1, 42, 2**40 + 7):
        for j in range(4):
            k = O.hash_key(seed, j)
            for _ in range(200):
                v = rng.getrandbits(32)
                assert fmix32_inverse(O.priority(seed, j, v)) ^ k == v
    p = O.priorities(1, 0, 1 << 20)
    assert np.unique(p).size == 1 << 20


def test_weight_reading_r1():
    # R1: p_j(v) = fmix32(v ^ K_j), K_j = fmix32(fold32(seed) + 0x9E3779B9 (j+1))
    for seed in (1, 42, (3 << 32) | 5):
        fold = (seed ^ (seed >> 32)) & M32
        for j in range(3):
            k = O.fmix32((fold + 0x9E3779B9 * (j + 1)) & M32)
            assert O.hash_key(seed, j) == k
            assert O.priority(seed, j, 12345) == O.fmix32(12345 ^ k)


def test_weight_values_used_by_golden():
    assert [O.priority(1, 0, v) for v in range(5)] == [
        0x70F6C6D8, 0xD2745AE2, 0xF6A49F81, 0xDB422EFE, 0xA577EB66]
    assert [O.priority(1, 1, v) for v in range(5)] == [
        0xBC154BEE, 0x64E66CB8, 0x33B403D5, 0x0CBA69A5, 0x806B0516]


# -------------------------------------------------------- golden colourings
@pytest.mark.parametrize("row", load_golden(), ids=lambda r: r[0])
def test_golden_hand_derived(row):
    name, n, edges, variant, expect = row
    g = G.csr_from_lists(n, edges)
    if variant == "maxmin":
        C = O.color_maxmin(g, 1)
    elif variant.startswith("multihash"):
        C = O.color_maxmin(g, 1, int(variant[len("multihash"):]))
    elif variant == "is_alg2":
        C = O.color_is_alg2(g, 1)
    elif variant == "jp_alg4":
        C = O.color_jp_alg4(g, 1)
    elif variant.startswith("hash_is"):
        C = O.color_hash_is(g, 1, int(variant[len("hash_is"):]))
    else:
        C = O.color_luby(g, 1)
    assert C.tolist() == expect


# ------------------------------------------------ Hash IS, Alg.6
@pytest.mark.parametrize("T", [0, 1, 3, 8])
def test_hash_is_proper_complete_and_bounded(T):
    for g in random_graphs(40, 60, seed0=700):
        n = g.n
        C, ncol, rounds = O.color_hash_is(g, 3, T, with_stats=True)
        assert O.check_proper(g, C) == 0
        assert (C != 0xFFFFFFFF).all()
        assert ncol == np.unique(C).size
        assert rounds <= 2 * n + 2  # R19: the heaviest uncoloured vertex wins within 2 rounds
        assert C.max(initial=0) < 2 * max(rounds, 1)


def test_hash_is_complete_graph_and_edgeless():
    for n in (1, 2, 5, 9):
        g = G.csr_from_lists(n, [(a, b) for a in range(n) for b in range(a + 1, n)])
        C, ncol, rounds = O.color_hash_is(g, 7, n, with_stats=True)
        # T >= Delta: every table holds both colours of each earlier round, so
        # each round takes the heaviest and lightest remaining vertex with new
        # colours: max-min's K_n closed form (n colours in ceil(n/2) rounds)
        assert ncol == n and rounds == (n + 1) // 2
        ref = O.color_maxmin(g, 7)
        if n % 2:  # the lone vertex of the last round: max-min's R9 gives it the
            ref[ref == n] = n - 1  # min colour 2k+1, Hash IS's R17 the max colour 2k
        assert C.tolist() == ref.tolist()
    g = G.csr_from_lists(6, [])
    assert O.color_hash_is(g, 7, 0).tolist() == [0] * 6


def test_hash_is_independent_of_row_order_and_duplicates():
    # R16: the proposal is the heaviest / lightest of the set, not Alg.6's
    # literal "last heavier neighbour", so entry order cannot matter
    rng = np.random.default_rng(3)
    for g in random_graphs(25, 80, seed0=900):
        ro, ci = g.row_offsets.numpy(), g.col_indices.numpy().copy()
        for v in range(g.n):
            seg = ci[ro[v]:ro[v + 1]].copy()
            rng.shuffle(seg)
            ci[ro[v]:ro[v + 1]] = seg
        h = G.Graph(g.n, g.row_offsets, torch.from_numpy(ci))
        for T in (0, 2):
            assert O.color_hash_is(g, 5, T).tolist() == O.color_hash_is(h, 5, T).tolist()


def test_hash_is_large_table_reuses_colours():
    # With T >= Delta a table holds every coloured neighbour's colour, so a
    # reused colour never clashes with an old neighbour: every vertex's colour
    # is either new in its round or absent from its neighbourhood -- and on
    # sparse random graphs the reuse must beat max-min's count.
    better = 0
    for g in random_graphs(30, 120, seed0=1100):
        deg = np.diff(g.row_offsets.numpy())
        T = int(deg.max(initial=0)) + 1
        C = O.color_hash_is(g, 11, T)
        assert O.check_proper(g, C) == 0
        better += np.unique(C).size <= np.unique(O.color_maxmin(g, 11)).size
    assert better >= 25


# ------------------------------------------------ Alg.2 / Alg.4
def _longest_decreasing_path(g, seed, key=None):
    # length (in vertices) of the longest strictly-decreasing-weight path
    # ending at each vertex: DP over vertices in decreasing weight order
    adj = adjacency(g)
    key = key or (lambda j, v: O.priority(seed, j, v))
    p = [key(0, v) for v in range(g.n)]
    depth = [0] * g.n
    for v in sorted(range(g.n), key=lambda x: p[x], reverse=True):
        depth[v] = 1 + max((depth[u] for u in adj[v] if p[u] > p[v]), default=0)
    return depth


def test_is_alg2_is_longest_decreasing_path():
    # Alg.2's colour of v = the iteration at which v is a local max among the
    # uncoloured = (longest decreasing-weight path ending at v) - 1
    for g in random_graphs(80, 40, seed0=11):
        for seed in (1, 5):
            C, R = O.color_is_alg2(g, seed, with_stats=True)
            d = _longest_decreasing_path(g, seed)
            assert C.tolist() == [x - 1 for x in d]
            assert R == (max(d) if g.n else 0)
            assert O.check_proper(g, C) == 0


def test_jp_alg4_properties():
    # Alg.4: proper; one colour per Alg.2 frontier; K_n -> ranks; edgeless ->
    # all 0; each frontier's colour is absent from its coloured neighbours and
    # every smaller colour is present among them (the first free colour)
    for n in (1, 6, 17):
        kn = G.csr_from_lists(n, [(a, b) for a in range(n) for b in range(a + 1, n)])
        p = O.priorities(3, 0, n)
        rank = {v: i for i, v in enumerate(sorted(range(n), key=lambda x: -int(p[x])))}
        assert O.color_jp_alg4(kn, 3).tolist() == [rank[v] for v in range(n)]
    assert O.color_jp_alg4(G.csr_from_lists(7, []), 2).tolist() == [0] * 7
    for g in random_graphs(80, 40, seed0=23):
        adj = adjacency(g)
        C = O.color_jp_alg4(g, 4)
        rounds = O.color_is_alg2(g, 4)  # iteration of each vertex
        assert O.check_proper(g, C) == 0
        for k in set(rounds.tolist()):
            F = [v for v in range(g.n) if rounds[v] == k]
            assert len({int(C[v]) for v in F}) == 1
            used = {int(C[u]) for v in F for u in adj[v] if rounds[u] < k}
            c = int(C[F[0]])
            assert c not in used and all(x in used for x in range(c))


# ------------------------------------------------ max-min / multi-hash oracle
@pytest.mark.parametrize("H", [1, 2, 3])
def test_maxmin_equals_literal_inplace_alg5(H):
    rng = random.Random(H)
    for g in random_graphs(60, 30, seed0=H):
        adj = adjacency(g)
        for seed in (1, 7):
            lit, iters = alg5_literal(g.n, adj, seed, H, rng)
            C, R, _ = O.color_maxmin(g, seed, H, with_stats=True)
            assert C.tolist() == lit
            assert R == iters


def test_maxmin_literal_on_cfg1_grid():
    g = G.grid2d(64, 64)
    lit, iters = alg5_literal(g.n, adjacency(g), 1, 1, random.Random(0))
    C, R, _ = O.color_maxmin(g, 1, with_stats=True)
    assert C.tolist() == lit and R == iters


@pytest.mark.parametrize("n", range(1, 13))
def test_complete_graph_closed_form(n):
    # K_n: each round colours exactly the max and the min of the remaining
    # vertices -> n distinct colours in ceil(n/2) rounds.
    g = G.csr_from_lists(n, [(a, b) for a in range(n) for b in range(a + 1, n)])
    C, R, nk = O.color_maxmin(g, 3, with_stats=True)
    assert R == (n + 1) // 2
    assert O.count_colors(C) == n
    assert nk == [n - 2 * k for k in range(R)]


def test_edgeless_and_star_closed_forms():
    assert O.color_maxmin(G.csr_from_lists(7, []), 9).tolist() == [1] * 7
    # star: the centre is coloured in round 0 (it is an extreme of the whole
    # graph) or all leaves are; in either case 2 rounds at most
    for seed in range(20):
        g = G.csr_from_lists(9, [(0, i) for i in range(1, 9)])
        C, R, _ = O.color_maxmin(g, seed, with_stats=True)
        assert R <= 2 and O.check_proper(g, C) == 0


def test_ncolors_2r_identity_and_proper():
    for g in random_graphs(80, 60, seed0=11):
        C, R, _ = O.color_maxmin(g, 5, with_stats=True)
        assert O.check_proper(g, C) == 0
        k = O.count_colors(C)
        assert k in (2 * R - 1, 2 * R)
        assert int(C.max()) < 2 * R


def test_multihash_h1_is_maxmin():
    for g in random_graphs(20, 50, seed0=3):
        assert (O.color_maxmin(g, 2, 1) == O.color_maxmin(g, 2)).all()


def test_certificate_accepts_and_rejects():
    rng = random.Random(8)
    for H in (1, 2, 4):
        for g in random_graphs(25, 40, seed0=20 + H):
            C = O.color_maxmin(g, 4, H)
            assert O.cert_maxmin(g, 4, H, C) == 0
            maxc = int(C.max())
            for _ in range(15):
                D = C.copy()
                v = rng.randrange(g.n)
                newc = rng.randrange(maxc + 3)
                if newc == D[v]:
                    continue
                D[v] = newc
                assert O.cert_maxmin(g, 4, H, D) != 0


def _first_improper(g, C):
    """1 + the first vertex (ascending) that is uncoloured or shares its colour
    with a neighbour, 0 if none: P:L40-44 written out with numpy."""
    ro, ci = g.row_offsets.numpy(), g.col_indices.numpy().astype(np.int64)
    src = np.repeat(np.arange(g.n), np.diff(ro))
    bad = C == O.UNCOLORED
    clash = C[src] == C[ci]
    bad[src[clash]] = True
    idx = np.flatnonzero(bad)
    return int(idx[0]) + 1 if idx.size else 0


def test_check_proper_rejects_mutations():
    """orc_check_proper (the problem definition) is pinned by what it
    must reject: on true colourings, recolouring one endpoint of a random edge
    to the other's colour and uncolouring a random vertex are both reported,
    at exactly the first offending vertex a numpy restatement finds; a
    colouring proper by construction (all colours distinct) is accepted."""
    rng = random.Random(31)
    for g in random_graphs(30, 60, seed0=90):
        C = O.color_maxmin(g, 5)
        assert O.check_proper(g, C) == 0 == _first_improper(g, C)
        assert O.check_proper(g, np.arange(g.n, dtype=np.uint32)) == 0
        ro, ci = g.row_offsets.numpy(), g.col_indices.numpy()
        for _ in range(10 if g.nnz else 0):
            e = rng.randrange(g.nnz)
            u = int(np.searchsorted(ro, e, side="right") - 1)
            w = int(ci[e])
            D = C.copy()
            D[u] = D[w]
            bad = O.check_proper(g, D)
            assert bad != 0 and bad - 1 <= min(u, w) and bad == _first_improper(g, D)
        v = rng.randrange(g.n)
        D = C.copy()
        D[v] = O.UNCOLORED
        bad = O.check_proper(g, D)
        assert bad != 0 and bad - 1 <= v and bad == _first_improper(g, D)


def test_chromatic_lower_bound():
    for g in random_graphs(40, 8, seed0=31):
        adj = adjacency(g)
        chi = chromatic_number(g.n, adj)
        for C in (O.color_maxmin(g, 1), O.color_maxmin(g, 1, 3), O.color_luby(g, 1),
                  O.color_greedy(g)):
            assert O.count_colors(C) >= chi


# ------------------------------------------------------------- Luby oracle
def test_luby_equals_greedy_in_priority_order_and_jp():
    for g in random_graphs(80, 40, seed0=41):
        adj = adjacency(g)
        for seed in (1, 3):
            C = O.color_luby(g, seed).tolist()
            order = sorted(range(g.n), key=lambda v: -O.priority(seed, 0, v))
            assert C == first_fit(g.n, adj, order)
            assert C == jones_plassmann(g.n, adj, seed)
            assert C == O.color_greedy_by_priority(g, seed).tolist()
            assert O.cert_mex(g, seed, np.array(C, dtype=np.uint32)) == 0


def test_luby_classes_are_maximal_independent_sets():
    for g in random_graphs(30, 50, seed0=51):
        adj = adjacency(g)
        C = O.color_luby(g, 2).tolist()
        delta = max((len(a) for a in adj), default=0)
        assert max(C, default=0) <= delta  # <= Delta + 1 colours
        for c in range(max(C, default=-1) + 1):
            cls = {v for v in range(g.n) if C[v] == c}
            residual = {v for v in range(g.n) if C[v] >= c}
            assert all(u not in cls for v in cls for u in adj[v])          # independent
            for v in residual - cls:                                        # maximal
                assert any(u in cls for u in adj[v])


def test_mex_certificate_rejects_mutations():
    rng = random.Random(3)
    for g in random_graphs(25, 40, seed0=61):
        C = O.color_luby(g, 5)
        for _ in range(10):
            D = C.copy()
            v = rng.randrange(g.n)
            D[v] = (int(D[v]) + 1 + rng.randrange(3)) % (int(C.max()) + 3)
            if D[v] != C[v]:
                assert O.cert_mex(g, 5, D) != 0


# ------------------------------------------------------------------ greedy
def test_greedy_bounds_and_closed_forms():
    for g in random_graphs(40, 60, seed0=71):
        adj = adjacency(g)
        C = O.color_greedy(g)
        delta = max((len(a) for a in adj), default=0)
        assert O.check_proper(g, C) == 0 and int(C.max(initial=0)) <= delta
        assert C.tolist() == first_fit(g.n, adj, range(g.n))
    # a bipartite grid in row-major order is a checkerboard: 2 colours
    assert O.count_colors(O.color_greedy(G.grid2d(64, 64))) == 2


def test_compact_colors():
    C = np.array([5, 1, 9, 1, 5], dtype=np.uint32)
    assert O.compact_colors(C).tolist() == [1, 0, 2, 0, 1]


def test_oracle_rejects_self_loops():
    g = G.Graph(2, __import__("torch").tensor([0, 2, 3]), __import__("torch").tensor([0, 1, 0],
                                                                                  dtype=__import__("torch").int32))
    with pytest.raises(O.OracleError):
        O.color_maxmin(g, 1)


# ------------------------------------------ N4: largest-degree-first (R21)
@pytest.mark.parametrize("H", [1, 2])
def test_ldf_maxmin_equals_literal_alg5_with_degree_keys(H):
    """LDF max-min = Alg.5 transcribed literally (in place, random thread
    order) with the priority replaced by the (degree, weight) tuple."""
    rng = random.Random(40 + H)
    for g in random_graphs(50, 30, seed0=60 + H):
        adj = adjacency(g)
        for seed in (2, 9):
            lit, iters = alg5_literal(g.n, adj, seed, H, rng, key=ldf_key(adj, seed))
            C, R, _ = O.color_maxmin(g, seed, H, with_stats=True, ldf=True)
            assert C.tolist() == lit and R == iters
            assert O.cert_maxmin(g, seed, H, C, ldf=True) == 0
            assert O.check_proper(g, C) == 0


def test_ldf_luby_alg2_alg4_closed_forms():
    """LDF Luby = first-fit greedy in decreasing (degree, weight) order (the
    classic largest-degree-first greedy) = Jones-Plassmann with those keys;
    LDF Alg.2 colour = longest decreasing-(degree, weight) path - 1; the mex
    certificate with LDF keys accepts them."""
    for g in random_graphs(60, 35, seed0=71):
        adj = adjacency(g)
        key = ldf_key(adj, 3)
        order = sorted(range(g.n), key=lambda v: key(0, v), reverse=True)
        C = O.color_luby(g, 3, ldf=True)
        assert C.tolist() == first_fit(g.n, adj, order) == jones_plassmann(g.n, adj, 3, key=key)
        assert (O.color_greedy_by_priority(g, 3, ldf=True) == C).all()
        assert O.cert_mex(g, 3, C, ldf=True) == 0
        C2, R2 = O.color_is_alg2(g, 3, with_stats=True, ldf=True)
        d = _longest_decreasing_path(g, 3, key=key)
        assert C2.tolist() == [x - 1 for x in d] and R2 == (max(d) if g.n else 0)
        C4 = O.color_jp_alg4(g, 3, ldf=True)
        assert O.check_proper(g, C4) == 0


def test_ldf_closed_forms_star_and_regular_graphs():
    """Star K_{1,s}: the centre has the largest degree, so under LDF it is the
    round-0 local max (colour 0) and every leaf a local min (colour 1), for
    every seed; Luby LDF colours the centre 0 and the leaves 1.  On regular
    graphs (cycle, K_n, hypercube) every degree ties, so LDF equals the plain
    random-priority colouring."""
    s = 40
    star = G.csr_from_lists(s + 1, [(0, i) for i in range(1, s + 1)])
    for seed in range(1, 8):
        assert O.color_maxmin(star, seed, ldf=True).tolist() == [0] + [1] * s
        assert O.color_luby(star, seed, ldf=True).tolist() == [0] + [1] * s
    d = 5
    cube = G.csr_from_lists(1 << d, [(v, v ^ (1 << b)) for v in range(1 << d) for b in range(d)
                                     if v < v ^ (1 << b)])
    for g in (G.csr_from_lists(9, [(i, (i + 1) % 9) for i in range(9)]),
              G.csr_from_lists(8, [(a, b) for a in range(8) for b in range(a + 1, 8)]), cube):
        for seed in (1, 4):
            assert (O.color_maxmin(g, seed, ldf=True) == O.color_maxmin(g, seed)).all()
            assert (O.color_luby(g, seed, ldf=True) == O.color_luby(g, seed)).all()
            assert (O.color_jp_alg4(g, seed, ldf=True) == O.color_jp_alg4(g, seed)).all()


def test_ldf_certificates_reject_mutations():
    rng = random.Random(77)
    for g in random_graphs(25, 40, seed0=81):
        C = O.color_maxmin(g, 6, ldf=True)
        L = O.color_luby(g, 6, ldf=True)
        assert O.cert_maxmin(g, 6, 1, C, ldf=True) == 0 and O.cert_mex(g, 6, L, ldf=True) == 0
        for _ in range(10):
            v = rng.randrange(g.n)
            D = C.copy()
            D[v] = (int(D[v]) + rng.randrange(1, 4)) % (int(C.max()) + 3)
            if D[v] != C[v]:
                assert O.cert_maxmin(g, 6, 1, D, ldf=True) != 0
            E = L.copy()
            E[v] = (int(E[v]) + rng.randrange(1, 4)) % (int(L.max()) + 3)
            if E[v] != L[v]:
                assert O.cert_mex(g, 6, E, ldf=True) != 0
