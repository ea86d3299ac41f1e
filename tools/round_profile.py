"""Per-round profile of one colouring (GC_PROFILE): kernel durations per round
and queue sizes, summarised in buckets.  Writes JSON to --out.

    python tools/round_profile.py --scale 24 [--mode event] --out gpurun_out/rounds.json
"""
import argparse
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--scale", type=int, default=24)
    ap.add_argument("--mode", default="event")
    ap.add_argument("--out", default="gpurun_out/rounds.json")
    a = ap.parse_args()
    g = G.rmat(a.scale, 16, seed=1, device="cuda")
    mode = {"event": gcb.MODE_EVENT, "sweep": gcb.MODE_SWEEP, "multi": gcb.MODE_EVENT_MULTI,
            "count": gcb.MODE_COUNT}[a.mode]
    out = torch.empty(g.n, dtype=torch.int32, device="cuda")
    hist_path = a.out + ".hist"
    if os.path.exists(hist_path):
        os.remove(hist_path)
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        h.color(1, gcb.MAXMIN, out, mode=mode)
        os.environ["GC_PROFILE_HIST"] = hist_path  # read by libgc at each profiled colouring
        _, k, st = h.color(1, gcb.MAXMIN, out, mode=mode, flags=gcb.PROFILE, stats=True,
                           trace_cap=1 << 15)
    R = st.rounds
    per = {gcb.MODE_EVENT: 3, gcb.MODE_EVENT_MULTI: 4, gcb.MODE_COUNT: 1}.get(mode, 2)
    lu = st.launch_us
    rows = []
    for r in range(R):
        rs = st.round_stats[16 * r: 16 * r + 16]
        # persistent kernel: per-phase times (ns) are in the round record
        if mode == gcb.MODE_COUNT:
            # [SL items, WL items, entries, coloured, round ns, max ns to flush start,
            #  max ns to targets set, max ns units done, max ns flush done,
            #  min ns units done (stored as ~ns), max cycles of one unit]
            rs = list(rs)
            if rs[9] < 0:
                rs[9] = -rs[9] - 1
            t = [rs[4] / 1e3]
        elif mode == gcb.MODE_EVENT:
            t = [x / 1e3 for x in rs[4:7]]
        else:
            t = lu[per * r: per * r + per]
        rows.append({"k": r, "us": t, "stats": rs})
    buckets = [(0, 1), (1, 2), (2, 10), (10, 100), (100, 500), (500, 1000), (1000, 2000),
               (2000, R)]
    summ = []
    for lo, hi in buckets:
        sel = rows[lo:min(hi, R)]
        if not sel:
            continue
        tot = [sum(x["us"][c] for x in sel) for c in range(per)]
        st4 = [sum(x["stats"][c] for x in sel) for c in range(16)]
        summ.append({"rounds": [lo, min(hi, R)], "us_by_class": tot, "us_total": sum(tot),
                     "stat_sums": st4, "us_per_round": sum(tot) / len(sel)})
    hist = None
    if os.path.exists(hist_path):
        with open(hist_path) as f:
            hist = json.loads(f.readlines()[-1])["hist"]
        names = ["seg scan (cycles)", "long-scan settle (cycles)", "warp eval (cycles)",
                 "notify segment (cycles)", "block work P1 (ns)", "block work P1b (ns)",
                 "block work P2 (ns)", "block work P3 (ns)"]
        hist = {names[i]: {f"2^{b}": hist[32 * i + b] for b in range(32) if hist[32 * i + b]}
                for i in range(8)}
        for nm, hh in hist.items():
            tot = sum(hh.values())
            print(nm, tot, hh)
    res = {"scale": a.scale, "mode": a.mode, "rounds": R, "n_colors": k, "ms": st.ms,
           "kernel_ms": st.kernel_ms, "buckets": summ, "op_histograms": hist,
           "top_rounds": sorted(rows, key=lambda x: -sum(x["us"]))[:25],
           "rows": [[x["k"], round(sum(x["us"]), 2)] + list(x["stats"][:4]) for x in rows]
           if mode == gcb.MODE_COUNT else None}
    os.makedirs(os.path.dirname(a.out) or ".", exist_ok=True)
    with open(a.out, "w") as f:
        json.dump(res, f, indent=1)
    for b in summ:
        print(json.dumps(b))
    print("top:", [(x["k"], [round(u, 1) for u in x["us"]], x["stats"]) for x in res["top_rounds"][:12]])


if __name__ == "__main__":
    main()
