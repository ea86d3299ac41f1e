# compute-sanitizer memcheck / racecheck / synccheck over tools/sanitize_run.py (every COUNT
# variant and mode on cfg1, cfg2, R-MAT s14, each checked against the oracle).
mkdir -p gpurun_out/san
for tool in memcheck racecheck synccheck; do
  timeout 1500 /usr/local/cuda/bin/compute-sanitizer --tool $tool --print-limit 20 python tools/sanitize_run.py cfg1 cfg2 s14 > gpurun_out/san/$tool.log 2>&1; echo "$tool rc=$?" >> gpurun_out/san/summary.txt
  tail -3 gpurun_out/san/$tool.log >> gpurun_out/san/summary.txt
done
