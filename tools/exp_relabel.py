"""Experiment (tools/, not product): does a degree-descending vertex relabel
speed up the COUNT kernel?  Times gc_color on R-MAT s24 as generated (labels
scattered by the seeded bijection) and on the same graph relabelled by degree
(hubs first).  Priorities follow the labels, so the two colourings differ;
only the timing and round counts are compared.

    python tools/exp_relabel.py [scale]
"""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402


def relabel(ro, ci, order):
    n = ro.numel() - 1
    deg = ro[1:] - ro[:-1]
    inv = torch.empty_like(order)
    inv[order] = torch.arange(n, device=ro.device, dtype=order.dtype)
    dn = deg[order]
    ron = torch.zeros(n + 1, dtype=torch.int64, device=ro.device)
    ron[1:] = torch.cumsum(dn, 0)
    m = int(ron[-1])
    src = torch.repeat_interleave(torch.arange(n, device=ro.device), dn)
    pos = torch.arange(m, device=ro.device) - ron[src]
    e = ro[order][src] + pos
    del src, pos
    cin = inv[ci[e].long()].to(torch.int32)
    return ron, cin


def timeit(name, ro, ci, n, reps=5, warm=2, variant=gcb.MAXMIN):
    out = torch.empty(n, dtype=torch.int32, device="cuda")
    with gcb.Graph(n, ro, ci, flags=gcb.BORROW_DEVICE) as h:
        ms = []
        for i in range(warm + reps):
            _, k, st = h.color(1, variant, out, mode=gcb.MODE_COUNT, stats=True)
            if i >= warm:
                ms.append(st.ms)
    print(json.dumps({"case": name, "ms_median": round(statistics.median(ms), 3), "rounds": st.rounds,
                      "n_colors": k}), flush=True)


def main():
    s = int(sys.argv[1]) if len(sys.argv) > 1 else 24
    g = G.rmat(s, 16, seed=1, device="cuda")
    ro, ci = g.row_offsets, g.col_indices
    n = g.n
    timeit(f"rmat s{s} as generated", ro, ci, n)
    deg = ro[1:] - ro[:-1]
    order = torch.sort(-deg, stable=True).indices
    ron, cin = relabel(ro, ci, order)
    timeit(f"rmat s{s} degree-descending labels", ron, cin, n)
    timeit(f"rmat s{s} degree-descending labels, luby", ron, cin, n, variant=gcb.LUBY_MIS)
    del ron, cin
    g2 = torch.randperm(n, device="cuda", generator=torch.Generator("cuda").manual_seed(5))
    ron, cin = relabel(ro, ci, g2)
    timeit(f"rmat s{s} random relabel (control)", ron, cin, n)


if __name__ == "__main__":
    main()
