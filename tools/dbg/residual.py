"""Useful vs walked entries per round, and residual graph size over rounds (R-MAT)."""
import sys, os, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import torch
import graphgen as G
import paper_conf_ipps_osamatybo19_b200 as gcb
scale = int(sys.argv[1]) if len(sys.argv) > 1 else 24
g = G.rmat(scale, 16, seed=1, device="cuda")
out = torch.empty(g.n, dtype=torch.int32, device="cuda")
with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
    h.color(1, gcb.MAXMIN, out, mode=gcb.MODE_COUNT)
rnd = (out.to(torch.int64) >> 1)
deg = g.row_offsets[1:] - g.row_offsets[:-1]
src = torch.repeat_interleave(torch.arange(g.n, device="cuda"), deg)
dst = g.col_indices.to(torch.int64)
ru, rw = rnd[src], rnd[dst]
R = int(rnd.max()) + 1
walked = torch.bincount(ru, minlength=R)
useful = torch.bincount(ru[rw > ru], minlength=R)
for lo, hi in [(0, 1), (1, 2), (2, 10), (10, 100), (100, 500), (500, 1000), (1000, 2000), (2000, R)]:
    print(f"rounds {lo}-{hi}: walked/round {float(walked[lo:hi].float().mean()):.0f} useful/round {float(useful[lo:hi].float().mean()):.0f}")
m = torch.minimum(ru, rw)   # edge (u,w) is in the residual at round r iff r <= min(round u, round w)
for r in [1, 2, 4, 8, 16, 32, 64, 128, 256, 512, 1024, 2048]:
    print(f"residual at round {r}: vertices {int((rnd >= r).sum())} entries {int((m >= r).sum())}")
