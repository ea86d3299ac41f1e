"""profiles/ncu_traffic.json from an `ncu --set full` capture of one colouring:
DRAM bytes (read + write) per launch of each COUNT kernel class, keyed by
workload, kernel class and the sha256 of the source that defines it (bench.py
only uses an entry whose sha matches the current source).

    python tools/ncu_traffic.py gpurun_out/prof.ncu-rep rmat-s24-maxmin
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from bench import source_sha  # noqa: E402


def main():
    rep, workload = sys.argv[1], sys.argv[2]
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True,
                         check=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr = rows[0]
    ki = hdr.index("Kernel Name")
    rd, wr, tm = (hdr.index("dram__bytes_read.sum"), hdr.index("dram__bytes_write.sum"),
                  hdr.index("gpu__time_duration.sum"))
    units = rows[1]
    scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
    cls = {}
    for r in rows[2:]:
        name = r[ki]
        c = ("k_count_persistent" if "k_count_persistent" in name else
             "counting pass" if any(x in name for x in ("k_count<", "k_count_hub<", "k_count_warp", "k_count_zero"))
             else None)
        if c is None:
            continue
        b = float(r[rd]) * scale[units[rd]] + float(r[wr]) * scale[units[wr]]
        e = cls.setdefault(c, {"bytes": 0.0, "launches": 0})
        e["bytes"] += b
        e["launches"] += 1
    path = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    try:
        d = json.load(open(path))
    except Exception:
        d = {}
    d = {k: v for k, v in d.items() if "|" in k}  # drop round-1 style keys
    for c, e in cls.items():
        per_step_launches = 1 if c == "k_count_persistent" else 2
        d[f"{workload}|{c}"] = {"kernel": c, "source_sha": source_sha(c),
                                "dram_bytes_per_launch": e["bytes"] / (e["launches"] / per_step_launches) / per_step_launches
                                if c == "k_count_persistent" else e["bytes"] / e["launches"],
                                "dram_bytes_per_step": e["bytes"] * per_step_launches / e["launches"],
                                "source": f"{os.path.basename(rep)} (ncu --set full --clock-control none, one colouring)"}
    json.dump(d, open(path, "w"), indent=1)
    print(json.dumps(d, indent=1))


if __name__ == "__main__":
    main()
