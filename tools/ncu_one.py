"""One colouring of the bench workload, for ncu captures (no timing here).
    python tools/ncu_one.py --mode event|sweep [--scale 24] [--warm]"""
import argparse, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import graphgen as G
import paper_conf_ipps_osamatybo19_b200 as gcb

ap = argparse.ArgumentParser()
ap.add_argument("--mode", default="event")
ap.add_argument("--scale", type=int, default=24)
ap.add_argument("--variant", default="maxmin")
ap.add_argument("--warm", action="store_true")
a = ap.parse_args()
mode = {"event": gcb.MODE_EVENT, "sweep": gcb.MODE_SWEEP, "multi": gcb.MODE_EVENT_MULTI,
        "count": gcb.MODE_COUNT, "auto": gcb.MODE_AUTO}[a.mode]
var = {"maxmin": gcb.MAXMIN, "luby": gcb.LUBY_MIS, "multihash": gcb.MULTIHASH(4),
       "hash": gcb.HASH_IS(8)}[a.variant]
g = G.rmat(a.scale, 16, seed=1, device="cuda")
torch.cuda.synchronize()
out = torch.empty(g.n, dtype=torch.int32, device="cuda")
with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
    if a.warm:
        h.color(1, var, out, mode=mode)
    _, k, st = h.color(1, var, out, mode=mode, stats=True)
torch.cuda.synchronize()
print("colours", k, "rounds", st.rounds, "ms", st.ms)
