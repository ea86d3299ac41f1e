"""End-of-round timeline of the COUNT kernel (needs a GC_PROF_FRESH=1 build via
GC_LIB_PATH): per round (max over blocks, us from the round start) the round
top, units done, fresh row offsets in, long-row list ready, flush start,
reservation back, flush end, and the round's total."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402

scale = int(sys.argv[1]) if len(sys.argv) > 1 else 24
g = G.rmat(scale, 16, seed=1, device="cuda")
out = torch.empty(g.n, dtype=torch.int32, device="cuda")
with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
    h.color(1, gcb.MAXMIN, out)
    _, k, st = h.color(1, gcb.MAXMIN, out, flags=gcb.PROFILE, stats=True, trace_cap=1 << 15)
R = st.rounds
rs = torch.tensor(st.round_stats[:16 * R], dtype=torch.float64).view(R, 16) / 1e3
print("ms", st.ms, "rounds", R)
for lo, hi in [(2, 10), (10, 100), (100, 1000), (1000, 2000), (2000, R)]:
    x = rs[lo:hi].mean(0)
    print(f"{lo}-{hi}: top {x[6]:.2f} units {x[7]:.2f} ro-in {x[14]:.2f} longs {x[15]:.2f} "
          f"flush-start {x[5]:.2f} resv {x[9]:.2f} flush-end {x[8]:.2f} round {x[4]:.2f}")
