timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "luby or golden or random or adversarial or cfg2 or s18" > gpurun_out/pt_jp.log 2>&1; echo rc=$? >> gpurun_out/pt_jp.log
timeout 300 python bench.py --variant luby --no-cpu-baseline --no-e2e > gpurun_out/bench_luby.json 2> gpurun_out/bench_luby.err
timeout 300 python tools/bench_configs.py > gpurun_out/configs.jsonl 2> gpurun_out/configs.err
