"""Experiment: COUNT kernel time on R-MAT s24 vs the number of persistent
blocks (GC_COUNT_BLOCKS) -- does a round's unit phase scale with SMs (per-SM
issue bound) or not (L2 / latency bound)?"""
import json, os, statistics, subprocess, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
if len(sys.argv) > 1:
    import torch
    import graphgen as G
    import paper_conf_ipps_osamatybo19_b200 as gcb
    g = G.rmat(int(sys.argv[1]), 16, seed=1, device="cuda")
    out = torch.empty(g.n, dtype=torch.int32, device="cuda")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        ms, cms = [], []
        for i in range(7):
            _, k, st = h.color(1, gcb.MAXMIN, out, stats=True)
            if i >= 2:
                ms.append(st.kernel_ms[0]); cms.append(st.kernel_ms[1])
    print(json.dumps({"blocks": os.environ.get("GC_COUNT_BLOCKS", "148"), "persistent_ms": statistics.median(ms), "counting_ms": statistics.median(cms),
                      "rounds": st.rounds}), flush=True)
else:
    for b in (37, 74, 111, 148):
        subprocess.run([sys.executable, __file__, "24"], env=dict(os.environ, GC_COUNT_BLOCKS=str(b)))
