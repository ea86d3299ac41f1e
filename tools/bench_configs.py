"""Time every BASELINE config / variant on one GPU (device time of gc_color_ex,
median of 5 after 2 warm-ups) and print one JSON line per case.

    python tools/bench_configs.py > gpurun_out/configs.jsonl
"""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402

MODES = {"event": gcb.MODE_EVENT, "sweep": gcb.MODE_SWEEP, "event-multi": gcb.MODE_EVENT_MULTI,
         "count": gcb.MODE_COUNT, "auto": gcb.MODE_AUTO}


def run(name, g, variant, vname, mode="event", reps=5, warm=2, loopback=0):
    out = torch.empty(g.n, dtype=torch.int32, device="cuda")
    if loopback:
        h = gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, loopback)
    else:
        h = gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE)
    with h:
        ms = []
        for i in range(warm + reps):
            _, k, st = h.color(1, variant, out, mode=MODES[mode], stats=True)
            if i >= warm:
                ms.append(st.ms)
    med = statistics.median(ms)
    rec = {"case": name, "variant": vname, "mode": mode if not loopback else f"loopback x{loopback}",
           "n": g.n, "nnz": g.nnz, "ms_median": round(med, 4), "gteps": round(g.nnz / med / 1e6, 3),
           "rounds": st.rounds, "inner_iterations": st.inner_iterations, "n_colors": k}
    print(json.dumps(rec), flush=True)


def main_hash():
    """the Hash IS (Alg.6, deterministic) on every config, T = 0 / 8."""
    dev = "cuda"
    for cfg, name in (("cfg1", "cfg1 grid 64x64"), ("cfg2", "cfg2 ER 2^20 d16"),
                      ("cfg3", "cfg3 mesh 128^3"), ("rgg", "N1 rgg_n_2_20"), ("cfg4", "cfg4 R-MAT s24")):
        g = G.rgg(20, seed=1, device=dev) if cfg == "rgg" else G.config_graph(cfg, dev)
        for T in (0, 8):
            run(name, g, gcb.HASH_IS(T), f"hash IS T={T}", "auto")
        run(name, g, gcb.MAXMIN, "maxmin", "auto")
        del g


def main():
    if os.environ.get("GC_ONLY") == "hash":
        return main_hash()
    dev = "cuda"
    g1 = G.config_graph("cfg1", dev)
    for m in ("count", "event", "sweep"):
        run("cfg1 grid 64x64", g1, gcb.MAXMIN, "maxmin", m)
    for m in ("count", "sweep"):
        run("cfg1 grid 64x64", g1, gcb.LUBY_MIS, "luby", m)
    g2 = G.config_graph("cfg2", dev)
    for m in ("count", "sweep"):
        run("cfg2 ER 2^20 d16", g2, gcb.LUBY_MIS, "luby", m)
    for m in ("count", "event", "sweep"):
        run("cfg2 ER 2^20 d16", g2, gcb.MAXMIN, "maxmin", m)
    del g2
    g3 = G.config_graph("cfg3", dev)
    for H in (1, 2, 4, 8):
        run("cfg3 mesh 128^3", g3, gcb.MULTIHASH(H), f"multihash H={H}", "sweep")
        run("cfg3 mesh 128^3", g3, gcb.MULTIHASH(H), f"multihash H={H}", "count")
    run("cfg3 mesh 128^3", g3, gcb.MAXMIN, "maxmin", "event")
    run("cfg3 mesh 128^3", g3, gcb.MAXMIN, "maxmin", "count")
    run("cfg3 mesh 128^3", g3, gcb.LUBY_MIS, "luby", "count")
    del g3
    gr = G.rgg(20, seed=1, device=dev)
    run("N1 rgg_n_2_20", gr, gcb.MAXMIN, "maxmin", "count")
    run("N1 rgg_n_2_20", gr, gcb.MAXMIN, "maxmin", "sweep")
    run("N1 rgg_n_2_20", gr, gcb.LUBY_MIS, "luby", "count")
    del gr
    g4 = G.config_graph("cfg4", dev)
    run("cfg4 R-MAT s24", g4, gcb.MAXMIN, "maxmin", "count")
    run("cfg4 R-MAT s24", g4, gcb.MAXMIN, "maxmin", "event")
    for H in (2, 4, 8):
        run("cfg4 R-MAT s24", g4, gcb.MULTIHASH(H), f"multihash H={H}", "count")
    run("cfg4 R-MAT s24", g4, gcb.LUBY_MIS, "luby", "count")
    if os.environ.get("GC_SLOW"):
        run("cfg4 R-MAT s24", g4, gcb.MAXMIN, "maxmin", "event-multi", reps=2, warm=1)
        run("cfg4 R-MAT s24", g4, gcb.MAXMIN, "maxmin", "sweep", reps=2, warm=1)
        run("cfg4 R-MAT s24", g4, gcb.LUBY_MIS, "luby", "sweep", reps=2, warm=1)
        run("cfg4 R-MAT s24", g4, gcb.MULTIHASH(4), "multihash H=4", "sweep", reps=2, warm=1)
    del g4
    g5 = G.rmat(22, 16, seed=1, device=dev)
    for p in (1, 2, 4, 8):
        run("R-MAT s22 partitioned", g5, gcb.MAXMIN, "maxmin", reps=2, warm=1, loopback=p)
    # G3_circuit-sized FEM stand-in (the paper's only printed runtime for this
    # path, Table II: 6.68 ms on a K40c for ~1.6M vertices / 7.7M edges)
    gm = G.mesh3d(117, 117, 117)
    run("mesh 117^3 (G3_circuit-sized)", gm, gcb.MAXMIN, "maxmin", "count")
    run("mesh 117^3 (G3_circuit-sized)", gm, gcb.MAXMIN, "maxmin", "sweep")


if __name__ == "__main__":
    main()
