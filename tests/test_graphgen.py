"""Seeded input generators (graphgen/): CSR invariants and workload shapes."""
import torch

import graphgen as G


def _check_csr(g):
    ro, ci = g.row_offsets, g.col_indices.to(torch.int64)
    assert ro[0] == 0 and ro[-1] == g.nnz and (ro[1:] >= ro[:-1]).all()
    rows = torch.repeat_interleave(torch.arange(g.n), ro[1:] - ro[:-1])
    assert (ci != rows).all(), "self-loop"
    assert (ci < g.n).all() and (ci >= 0).all()
    fwd = torch.unique(rows * g.n + ci)
    assert fwd.numel() == g.nnz, "duplicate entries"
    bwd = torch.sort(ci * g.n + rows).values
    assert torch.equal(fwd, bwd), "not symmetric"
    # rows sorted ascending
    d = ci[1:] - ci[:-1]
    same_row = rows[1:] == rows[:-1]
    assert (d[same_row] > 0).all()


def test_grid_and_mesh_exact_sizes():
    g = G.grid2d(64, 64)
    assert (g.n, g.nnz) == (4096, 16128)
    _check_csr(g)
    m = G.mesh3d(16, 16, 16)
    assert m.nnz == 2 * 3 * 16 * 16 * 15
    _check_csr(m)


def test_er_and_rmat_invariants_and_determinism():
    e = G.erdos_renyi(4096, 8 * 4096, seed=1)
    _check_csr(e)
    assert abs(e.nnz / e.n - 16) < 0.5
    r = G.rmat(12, 16, seed=1)
    _check_csr(r)
    r2 = G.rmat(12, 16, seed=1)
    assert torch.equal(r.col_indices, r2.col_indices)
    assert not torch.equal(G.rmat(12, 16, seed=2).row_offsets, r.row_offsets)
    deg = r.degrees()
    assert int(deg.max()) > 20 * float(deg.float().mean())  # power law: hubs


def test_rgg_degree_law_matches_table1():
    # Table I: rgg_n_2_15 avg degree 9.78, 2_16 10.44, 2_17 11.11
    for scale, paper in ((15, 9.78), (16, 10.44), (17, 11.11)):
        g = G.rgg(scale, seed=1)
        if scale == 15:
            _check_csr(g)
        assert abs(g.nnz / g.n - paper) / paper < 0.03


def test_label_permutation_is_bijective():
    x = torch.arange(1 << 12)
    y = G._label_permutation(x, 12, seed=9)
    assert torch.equal(torch.sort(y).values, x)


def test_rmat_built_by_pieces_is_identical():
    """The range-by-range build (used for cfg5, s27) yields the same CSR."""
    a = G.rmat(13, 16, seed=4)
    for pieces in (2, 3, 8):
        b = G.rmat(13, 16, seed=4, pieces=pieces)
        assert torch.equal(a.row_offsets, b.row_offsets) and torch.equal(a.col_indices, b.col_indices)
