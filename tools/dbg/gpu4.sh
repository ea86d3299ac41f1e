timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q -m gpu > gpurun_out/pt_mh.log 2>&1; echo rc=$? >> gpurun_out/pt_mh.log
timeout 300 python bench.py --variant multihash --hashes 4 --no-cpu-baseline --no-e2e > gpurun_out/bench_mh.json 2> gpurun_out/bench_mh.err
timeout 600 python tools/bench_configs.py > gpurun_out/configs.jsonl 2> gpurun_out/configs.err
