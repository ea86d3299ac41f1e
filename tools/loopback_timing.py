"""Partitioned COUNT rounds through the loopback transport (P partitions on one
GPU, the same kernels and exchange protocol as across GPUs) vs the single-GPU
path: device ms per colouring (median of 5) on R-MAT s<scale>.

    python tools/loopback_timing.py 22 > profiles/r02_loopback_count.jsonl
"""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402


def timed(h, n, reps=5, warm=2):
    out = torch.empty(n, dtype=torch.int32, device="cuda")
    ms = []
    for i in range(warm + reps):
        _, k, st = h.color(1, gcb.MAXMIN, out, stats=True)
        if i >= warm:
            ms.append(st.ms)
    return statistics.median(ms), st.rounds, k, out


def main():
    scale = int(sys.argv[1]) if len(sys.argv) > 1 else 22
    g = G.rmat(scale, 16, seed=1, device="cuda")
    with gcb.Graph(g.n, g.row_offsets, g.col_indices, flags=gcb.BORROW_DEVICE) as h:
        ms1, R, k, ref = timed(h, g.n)
    rounds_mode = "host" if os.environ.get("GC_DIST_HOST_ROUNDS") == "1" else "device"
    print(json.dumps({"graph": f"rmat s{scale}", "path": "single GPU", "ms": round(ms1, 3), "rounds": R}), flush=True)
    for parts in (1, 2, 4, 8):
        with gcb.loopback_graph(g.n, g.row_offsets, g.col_indices, parts) as h:
            ms, R2, k2, out = timed(h, g.n)
        print(json.dumps({"graph": f"rmat s{scale}", "path": f"loopback P={parts}", "rounds_driven_by": rounds_mode,
                          "ms": round(ms, 3), "rounds": R2, "vs_single_gpu": round(ms / ms1, 2),
                          "equal_to_single_gpu": bool(torch.equal(out, ref))}), flush=True)


if __name__ == "__main__":
    main()
