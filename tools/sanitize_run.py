"""One colouring per (config, variant, mode) on small graphs, for
compute-sanitizer (memcheck / racecheck / synccheck).  Each colouring is
checked against the oracle, so a tool-induced schedule change that altered a
result would show up as a mismatch.

    compute-sanitizer --tool memcheck python tools/sanitize_run.py
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402
import torch  # noqa: E402

import graphgen as G  # noqa: E402
import oracle as O  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402

CASES = [
    ("maxmin", gcb.MAXMIN, gcb.MODE_COUNT, lambda g: O.color_maxmin(g, 1)),
    ("maxmin", gcb.MAXMIN, gcb.MODE_SWEEP, lambda g: O.color_maxmin(g, 1)),
    ("maxmin", gcb.MAXMIN, gcb.MODE_EVENT, lambda g: O.color_maxmin(g, 1)),
    ("multihash4", gcb.MULTIHASH(4), gcb.MODE_COUNT, lambda g: O.color_maxmin(g, 1, 4)),
    ("luby", gcb.LUBY_MIS, gcb.MODE_COUNT, lambda g: O.color_luby(g, 1)),
    ("luby", gcb.LUBY_MIS, gcb.MODE_SWEEP, lambda g: O.color_luby(g, 1)),
    ("is_alg2", gcb.IS_ALG2, gcb.MODE_COUNT, lambda g: O.color_is_alg2(g, 1)),
    ("jp_alg4", gcb.JP_ALG4, gcb.MODE_COUNT, lambda g: O.color_jp_alg4(g, 1)),
    ("hash_is8", gcb.HASH_IS(8), gcb.MODE_AUTO, lambda g: O.color_hash_is(g, 1, 8)),
    ("maxmin_ldf", gcb.LDF(gcb.MAXMIN), gcb.MODE_COUNT, lambda g: O.color_maxmin(g, 1, ldf=True)),
    ("luby_ldf", gcb.LDF(gcb.LUBY_MIS), gcb.MODE_COUNT, lambda g: O.color_luby(g, 1, ldf=True)),
]


def main():
    which = sys.argv[1:] or ["cfg1", "cfg2"]
    for cfg in which:
        g = G.config_graph(cfg) if cfg.startswith("cfg") else G.rmat(int(cfg[1:]), 16, seed=1)
        with gcb.Graph(g.n, g.row_offsets, g.col_indices) as h:
            for name, v, mode, ref in CASES:
                out = torch.empty(g.n, dtype=torch.int32, device="cuda")
                _, k, st = h.color(1, v, out, mode=mode, stats=True)
                ok = (out.cpu().numpy().view(np.uint32) == ref(g)).all()
                print(f"{cfg} {name} mode {st.mode_used}: colours {k} rounds {st.rounds} "
                      f"{'ok' if ok else 'MISMATCH'}", flush=True)
                assert ok
        # the partitioned kernel (device-driven rounds), 2 and 3 partitions on this GPU
        for parts in (2, 3):
            with gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, parts) as h:
                out = torch.empty(g.n, dtype=torch.int32, device="cuda")
                _, k, st = h.color(1, gcb.MAXMIN, out, stats=True)
                ok = (out.cpu().numpy().view(np.uint32) == O.color_maxmin(g, 1)).all()
                print(f"{cfg} maxmin loopback P={parts}: colours {k} rounds {st.rounds} "
                      f"{'ok' if ok else 'MISMATCH'}", flush=True)
                assert ok


if __name__ == "__main__":
    main()
