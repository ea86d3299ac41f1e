"""Per round: decrements per vertex (max / top), from a COUNT-mode colouring of R-MAT."""
import sys, os, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
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
R = int(rnd.max()) + 1
key = rnd[src] * g.n + dst          # decrements of dst in round rnd[src]
key, cnt = torch.unique(key, return_counts=True)
kr = key // g.n
mx = torch.zeros(R, dtype=torch.int64, device="cuda").scatter_reduce(0, kr, cnt, "amax")
tot = torch.zeros(R, dtype=torch.int64, device="cuda").scatter_add(0, kr, cnt)
res = {"rounds": R, "max_per_round": mx.tolist(), "entries_per_round": tot.tolist()}
for lo, hi in [(0, 1), (1, 2), (2, 10), (10, 100), (100, 500), (500, 1000), (1000, 2000), (2000, R)]:
    print(lo, hi, "mean max-decrements-per-vertex", float(mx[lo:hi].float().mean()), "max", int(mx[lo:hi].max()),
          "mean entries", float(tot[lo:hi].float().mean()))
json.dump(res, open("gpurun_out/contention.json", "w"))
