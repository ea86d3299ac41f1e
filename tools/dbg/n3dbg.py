import sys, random
sys.path.insert(0, '.')
import numpy as np, torch
import graphgen as G, oracle as O, paper_conf_ipps_osamatybo19_b200 as gcb
rng = random.Random(1 * 7 + len("is_alg2"))
for i in range(120):
    n = rng.randint(0, 300)
    p = rng.choice([0.0, 0.01, 0.05, 0.2, 0.5])
    g = G.random_graph(n, p, seed=1000 * 1 + i)
    seed = rng.getrandbits(64)
    for var, fn in ((gcb.IS_ALG2, O.color_is_alg2), (gcb.JP_ALG4, O.color_jp_alg4), (gcb.LUBY_MIS, O.color_luby)):
        ref = fn(g, seed)
        with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
            out = torch.empty(g.n, dtype=torch.int32)
            try:
                _, k, st = h.color(seed, var, out, stats=True, mode=gcb.MODE_COUNT)
                C = out.numpy().view(np.uint32)
                if not (C == ref).all():
                    bad = np.nonzero(C != ref)[0]
                    print("MISMATCH", var, i, n, p, bad[:10], C[bad[:10]], ref[bad[:10]])
            except Exception as e:
                deg = np.diff(g.row_offsets.numpy())
                print("ERR", var, i, n, p, "maxdeg", deg.max() if n else 0, e)
