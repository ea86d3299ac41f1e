set -x
mkdir -p gpurun_out/san
for tool in memcheck racecheck synccheck; do
  timeout 1500 /usr/local/cuda/bin/compute-sanitizer --tool $tool --print-limit 20 python tools/sanitize_run.py cfg1 cfg2 s14 > gpurun_out/san/$tool.log 2>&1; echo "$tool rc=$?" >> gpurun_out/san/summary.txt
  tail -3 gpurun_out/san/$tool.log >> gpurun_out/san/summary.txt
done
GC_SLOW_TESTS=1 timeout 2400 python -m pytest tests/test_gpu_parity.py -q -k "elementwise" --durations=3 > gpurun_out/san/slow_s24.log 2>&1; echo "slow rc=$?" >> gpurun_out/san/summary.txt
