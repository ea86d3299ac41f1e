"""SURVEY N1 / the paper's scalability study (Fig.3):
rgg_n_2_{15..24} (Table I), every IS variant on one B200.

Per scale and variant: device ms of one colouring (gc_color_ex, median of 5
after 2 warm-ups), GTEPS (directed entries / ms), rounds, colours.  The paper
compares the fastest IS implementations of its two frameworks: Gunrock IS
(max-min, our GC_MAXMIN) and GraphBLAST IS (Alg.2, our GC_IS_ALG2), and
reports 1.14x fewer colours for Gunrock; the line
"summary" gives our colour ratio per scale and its geometric mean.

    python tools/rgg_sweep.py > profiles/r02_rgg_sweep.jsonl
"""
import json
import math
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402

VARIANTS = [("maxmin (Gunrock IS, Alg.5)", gcb.MAXMIN), ("is_alg2 (GraphBLAST IS, Alg.2)", gcb.IS_ALG2),
            ("luby (GraphBLAST MIS, Alg.2+3)", gcb.LUBY_MIS), ("jp_alg4 (GraphBLAST JP, Alg.4)", gcb.JP_ALG4),
            ("hash_is8 (Gunrock Hash, Alg.6)", gcb.HASH_IS(8)), ("multihash4", gcb.MULTIHASH(4))]


def main():
    lo, hi = (int(sys.argv[1]), int(sys.argv[2])) if len(sys.argv) > 2 else (15, 24)
    ratios = []
    for s in range(lo, hi + 1):
        g = G.rgg(s, seed=1, device="cuda")
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        res = {}
        with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
            for name, v in VARIANTS:
                ms = []
                for i in range(7):
                    _, k, st = h.color(1, v, out, stats=True)
                    if i >= 2:
                        ms.append(st.ms)
                med = statistics.median(ms)
                res[name] = k
                print(json.dumps({"graph": f"rgg_n_2_{s}", "n": g.n, "nnz": g.nnz,
                                  "avg_degree": round(g.nnz / g.n, 2), "variant": name,
                                  "ms_median": round(med, 4), "gteps": round(g.nnz / med / 1e6, 3),
                                  "rounds": st.rounds, "n_colors": k, "mode_used": st.mode_used}),
                      flush=True)
        r = res["is_alg2 (GraphBLAST IS, Alg.2)"] / res["maxmin (Gunrock IS, Alg.5)"]
        ratios.append(r)
        del g, out
        torch.cuda.empty_cache()
    print(json.dumps({"summary": "colours GraphBLAST IS (Alg.2) / Gunrock IS (max-min) per scale",
                      "scales": list(range(lo, hi + 1)), "ratios": [round(x, 3) for x in ratios],
                      "geomean": round(math.exp(sum(map(math.log, ratios)) / len(ratios)), 3),
                      "paper": "1.14x fewer colours for Gunrock IS (PAPER.md:1003-1004, Fig.3d)"}))


if __name__ == "__main__":
    main()
