"""Summarise ncu outputs into profiles/ (committed evidence).

    python tools/ncu_summary.py launches gpurun_out/launches_event.csv > profiles/...md
    python tools/ncu_summary.py full gpurun_out/prof_event.ncu-rep > profiles/...md

`launches`: per-kernel totals of a `--metrics gpu__time_duration.sum` launch list
(cold-cache, serialised: compare shares, not absolutes).
`full`: the key metrics of a `--set full` capture (DRAM bytes, throughput,
occupancy, registers, stall reasons)."""
import csv
import re
import io
import subprocess
import sys
from collections import defaultdict


def kname(full):
    """'void gc::<unnamed>::k_sweep<1, false>(gc::SweepArgs)' -> 'k_sweep<1, false>'."""
    head = full.split("(")[0]
    m = re.search(r"(\w+)(<[^<>]*>)?\s*$", head)
    return (m.group(1) + (m.group(2) or "")) if m else head


def launches(path):
    rows = list(csv.reader(open(path)))
    hdr_i = next(i for i, r in enumerate(rows) if "Kernel Name" in r)
    hdr = rows[hdr_i]
    ki, mi, vi = hdr.index("Kernel Name"), hdr.index("Metric Name"), hdr.index("Metric Value")
    ui = hdr.index("Metric Unit") if "Metric Unit" in hdr else None
    tot = defaultdict(float)
    cnt = defaultdict(int)
    for r in rows[hdr_i + 1:]:
        if len(r) <= vi or r[mi] != "gpu__time_duration.sum":
            continue
        v = float(r[vi].replace(",", ""))
        unit = r[ui] if ui is not None else "ns"
        v *= {"ns": 1e-3, "usecond": 1.0, "us": 1.0, "msecond": 1e3, "ms": 1e3, "nsecond": 1e-3}.get(unit, 1e-3)
        name = kname(r[ki])
        tot[name] += v
        cnt[name] += 1
    ours = {k: v for k, v in tot.items() if k.startswith("k_")}
    allsum = sum(tot.values())
    oursum = sum(ours.values())
    print(f"source: `{path}` (ncu --metrics gpu__time_duration.sum --clock-control none)\n")
    print(f"all kernels: {allsum/1e3:.3f} ms over {sum(cnt.values())} launches; libgc kernels: "
          f"{oursum/1e3:.3f} ms over {sum(cnt[k] for k in ours)} launches\n")
    print("| kernel | launches | total ms | share of libgc time | avg us |")
    print("|---|---:|---:|---:|---:|")
    for k, v in sorted(ours.items(), key=lambda x: -x[1]):
        print(f"| `{k}` | {cnt[k]} | {v/1e3:.3f} | {100*v/max(oursum,1e-9):.1f}% | {v/cnt[k]:.2f} |")


KEYS = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "dram__throughput.avg.pct_of_peak_sustained_elapsed", "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed",
        "lts__t_bytes.sum", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
        "sm__warps_active.avg.pct_of_peak_sustained_active", "launch__registers_per_thread",
        "launch__grid_size", "launch__block_size", "sm__inst_executed.sum",
        "l1tex__t_sector_hit_rate.pct", "lts__t_sector_hit_rate.pct",
        "smsp__average_warp_latency_issue_stalled_long_scoreboard",
        "smsp__average_warps_issue_stalled_long_scoreboard_per_issue_active.ratio",
        "smsp__average_warps_issue_stalled_barrier_per_issue_active.ratio",
        "smsp__average_warps_issue_stalled_membar_per_issue_active.ratio",
        "smsp__average_warps_issue_stalled_sleeping_per_issue_active.ratio",
        "smsp__average_warps_issue_stalled_lg_throttle_per_issue_active.ratio"]


def full(path):
    out = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True,
                         text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr, units = rows[0], rows[1]
    print(f"source: `{path}` (ncu --set full --clock-control none --import-source on)\n")
    for r in rows[2:]:
        name = r[hdr.index("Kernel Name")] if "Kernel Name" in hdr else "?"
        print(f"### `{kname(name)}`\n")
        print("| metric | value | unit |")
        print("|---|---:|---|")
        for k in KEYS:
            if k in hdr:
                i = hdr.index(k)
                print(f"| {k} | {r[i]} | {units[i]} |")
        print()


if __name__ == "__main__":
    {"launches": launches, "full": full}[sys.argv[1]](sys.argv[2])
