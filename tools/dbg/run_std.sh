timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -m gpu > gpurun_out/pt_count.log 2>&1; echo rc=$? >> gpurun_out/pt_count.log
timeout 300 python bench.py --mode count --no-cpu-baseline --no-e2e > gpurun_out/bench_count.json 2> gpurun_out/bench_count.err
timeout 200 python tools/round_profile.py --scale 24 --mode count --out gpurun_out/rounds_count.json > gpurun_out/rounds_count.log 2>&1
