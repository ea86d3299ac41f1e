"""Debug: reproduce test_random_small_graphs[maxmin-1] case i and diff COUNT mode vs oracle."""
import random, sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np, torch
import graphgen as G, oracle as O
import paper_conf_ipps_osamatybo19_b200 as gcb
rng = random.Random(1 * 7 + len("maxmin"))
cases = []
for i in range(120):
    n = rng.randint(0, 300); p = rng.choice([0.0, 0.01, 0.05, 0.2, 0.5])
    g = G.random_graph(n, p, seed=1000 * 1 + i); seed = rng.getrandbits(64)
    for mode in [1, 2, 3, 4]:
        rng.choice([0, 1, 4, 64]); rng.choice([0, 2, 40, 1 << 20]); rng.choice([0, 1, 3])
    cases.append((g, seed))
bad = 0
for i, (g, seed) in enumerate(cases):
    ref = O.color_maxmin(g, seed)
    with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
        out = torch.empty(g.n, dtype=torch.int32)
        for rep in range(3):
            h.color(seed, gcb.MAXMIN, out, mode=gcb.MODE_COUNT)
            C = out.numpy().view(np.uint32)
            d = np.nonzero(C != ref)[0]
            if len(d):
                bad += 1
                deg = (g.row_offsets[1:] - g.row_offsets[:-1]).numpy()
                print("case", i, "rep", rep, "n", g.n, "ndiff", len(d), [(int(v), int(C[v]), int(ref[v]), int(deg[v])) for v in d[:10]])
print("bad", bad)
