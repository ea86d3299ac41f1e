"""SURVEY N4 / PAPER.md:1090-1098: largest-degree-first vs random priorities.
"With power law graphs, is possible that a random weight initialization would
perform worse than largest-degree first" -- per workload and IS variant:
rounds, colours and device ms (median of 5) with random weights (R1) and with
(degree, weight) keys (R21), one B200.

    python tools/ldf_compare.py > profiles/r02_ldf_compare.jsonl
"""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402

VARIANTS = [("maxmin", gcb.MAXMIN), ("luby", gcb.LUBY_MIS), ("is_alg2", gcb.IS_ALG2), ("jp_alg4", gcb.JP_ALG4)]


def main():
    cases = [("cfg4 R-MAT s24", lambda: G.config_graph("cfg4", device="cuda")),
             ("cfg2 ER 2^20 d16", lambda: G.config_graph("cfg2", device="cuda")),
             ("cfg3 mesh 128^3", lambda: G.config_graph("cfg3", device="cuda")),
             ("rgg_n_2_20", lambda: G.rgg(20, seed=1, device="cuda")),
             ("R-MAT s20", lambda: G.rmat(20, 16, seed=1, device="cuda"))]
    for name, mk in cases:
        g = mk()
        out = torch.empty(g.n, dtype=torch.int32, device="cuda")
        with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
            for vname, v in VARIANTS:
                rec = {"graph": name, "n": g.n, "nnz": g.nnz, "variant": vname}
                for tag, code in (("random", v), ("ldf", gcb.LDF(v))):
                    ms = []
                    for i in range(7):
                        _, k, st = h.color(1, code, out, stats=True, mode=gcb.MODE_COUNT)
                        if i >= 2:
                            ms.append(st.ms)
                    rec[tag] = {"rounds": st.rounds, "n_colors": k, "ms_median": round(statistics.median(ms), 3)}
                rec["colour_ratio_random_over_ldf"] = round(rec["random"]["n_colors"] / rec["ldf"]["n_colors"], 3)
                print(json.dumps(rec), flush=True)
        del g, out
        torch.cuda.empty_cache()


if __name__ == "__main__":
    main()
