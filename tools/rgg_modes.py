"""Experiment: max-min on rgg_n_2_<s> in each mode, with the per-round times
of the COUNT kernel (GC_PROFILE)."""
import os, sys, statistics
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import graphgen as G
import paper_conf_ipps_osamatybo19_b200 as gcb
s = int(sys.argv[1]) if len(sys.argv) > 1 else 24
g = G.rgg(s, seed=1, device="cuda")
out = torch.empty(g.n, dtype=torch.int32, device="cuda")
with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
    for name, m in (("count", gcb.MODE_COUNT), ("sweep", gcb.MODE_SWEEP), ("event", gcb.MODE_EVENT)):
        ms = []
        for i in range(4):
            _, k, st = h.color(1, gcb.MAXMIN, out, mode=m, stats=True)
            if i: ms.append(st.ms)
        print(name, "ms", round(statistics.median(ms), 3), "rounds", st.rounds, "kernel_ms", [round(x, 3) for x in st.kernel_ms])
    _, k, st = h.color(1, gcb.MAXMIN, out, mode=gcb.MODE_COUNT, flags=gcb.PROFILE, stats=True, trace_cap=1 << 12)
    R = st.rounds
    rs = torch.tensor(st.round_stats[:16 * R], dtype=torch.float64).view(R, 16)
    for k in range(R):
        x = rs[k]
        print(f"round {k}: SL {int(x[0])} WL {int(x[1])} entries {int(x[2])} coloured {int(x[3])} us {x[4]/1e3:.1f} units {x[7]/1e3:.1f} flushend {x[8]/1e3:.1f}")
