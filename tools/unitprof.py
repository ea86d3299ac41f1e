"""Per-round WL-unit latency breakdown (needs a GC_PROF_UNIT=1 build via GC_LIB_PATH)."""
import sys, os, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import graphgen as G
import paper_conf_ipps_osamatybo19_b200 as gcb
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
from exp_relabel import relabel
scale = int(sys.argv[1]) if len(sys.argv) > 1 else 24
g = G.rmat(scale, 16, seed=1, device="cuda")
CL = 1.965e3  # cycles per us at max clock

def prof(name, ro, ci):
    out = torch.empty(g.n, dtype=torch.int32, device="cuda")
    with gcb.Graph(g.n, ro, ci, flags=gcb.BORROW_DEVICE) as h:
        h.color(1, gcb.MAXMIN, out, mode=gcb.MODE_COUNT)
        _, k, st = h.color(1, gcb.MAXMIN, out, mode=gcb.MODE_COUNT, flags=gcb.PROFILE, stats=True, trace_cap=1 << 15)
    R = st.rounds
    rs = torch.tensor(st.round_stats[:16 * R], dtype=torch.float64).view(R, 16)
    print(name, "ms", st.ms, "rounds", R)
    for lo, hi in [(2, 10), (10, 100), (100, 1000), (1000, 2000), (2000, R)]:
        x = rs[lo:hi]
        nw = x[:, 1].sum()
        print(f"  {lo}-{hi}: us/round {x[:,4].mean()/1e3:.2f} WL/round {x[:,1].mean():.0f} | max item {x[:,12].mean()/CL:.2f} max col {x[:,14].mean()/CL:.2f} max atom {x[:,15].mean()/CL:.2f} max WL unit {x[:,10].mean()/CL:.2f} max SL unit {x[:,13].mean()/CL:.2f} | mean to-col {x[:,11].sum()/nw/CL:.2f} mean atom {x[:,9].sum()/nw/CL:.2f} | top {x[:,6].mean()/1e3:.2f} units done {x[:,7].mean()/1e3:.2f} publish {x[:,5].mean()/1e3:.2f} poll done {x[:,8].mean()/1e3:.2f}")

prof("as generated", g.row_offsets, g.col_indices)
if "quick" in sys.argv:
    sys.exit(0)
deg = g.row_offsets[1:] - g.row_offsets[:-1]
order = torch.sort(-deg, stable=True).indices
ron, cin = relabel(g.row_offsets, g.col_indices, order)
prof("degree-descending", ron, cin)
n = g.n
rank = torch.empty_like(order); rank[order] = torch.arange(n, device="cuda")
# spread: hot vertices (low degree-rank) dealt over 256 interleaved regions (different L2 lines / slices)
S = 256
newid = (rank % S) * (n // S) + rank // S
order2 = torch.empty_like(order); order2[newid] = torch.arange(n, device="cuda")
del ron, cin
ron, cin = relabel(g.row_offsets, g.col_indices, order2)
prof("degree-rank spread over 256 regions", ron, cin)
