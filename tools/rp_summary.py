"""Summary of a tools/round_profile.py JSON: kernel classes, round 0/1, per-bucket us/round."""
import json, sys, statistics as S
d = json.load(open(sys.argv[1]))
print("ms", round(d["ms"], 3), "kernel_ms", [round(x, 3) for x in d["kernel_ms"]])
rows = d["rows"]
for lo, hi in [(0, 1), (1, 2), (2, 10), (10, 100), (100, 1000), (1000, 2000), (2000, len(rows))]:
    rr = [r for r in rows if lo <= r[0] < hi]
    if rr:
        print(lo, hi, "us", round(S.mean(r[1] for r in rr), 2), "SL", int(S.mean(r[2] for r in rr)),
              "WL", int(S.mean(r[3] for r in rr)), "entries", int(S.mean(r[4] for r in rr)),
              "coloured", int(S.mean(r[5] for r in rr)))
