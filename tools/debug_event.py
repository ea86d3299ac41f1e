"""Colour R-MAT graphs in one mode and compare with the oracle (debug aid)."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import graphgen as G, oracle as O
import paper_conf_ipps_osamatybo19_b200 as gcb

mode = {"event": gcb.MODE_EVENT, "multi": gcb.MODE_EVENT_MULTI, "sweep": gcb.MODE_SWEEP}[sys.argv[1].split(":")[0]]
for s in [int(x) for x in sys.argv[2:]]:
    g = G.rmat(s, 16, seed=1)
    ref = O.color_maxmin(g, 1)
    with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
        out = torch.empty(g.n, dtype=torch.int32)
        try:
            _, k, st = h.color(1, gcb.MAXMIN, out, mode=mode, stats=True)
        except gcb.GCError as e:
            print("scale", s, "ERROR", e, flush=True)
            break
        C = out.numpy().view(np.uint32)
        bad = np.nonzero(C != ref)[0]
        print("scale", s, "rounds", st.rounds, "colours", k, "mismatches", bad.size, bad[:10], flush=True)
