# One full GPU measurement pass (tests, smoke, bench, ncu launch list + full capture, configs, per-round profile):
#   bash tools/dbg/gpu.sh 4000 "bash tools/dbg/full_run.sh"
timeout 1500 python -m pytest tests/ -x -q -m gpu > gpurun_out/pt_all.log 2>&1; echo rc=$? >> gpurun_out/pt_all.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo rc=$? >> gpurun_out/smoke.log
timeout 600 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err
timeout 600 python bench.py --variant luby --no-cpu-baseline > gpurun_out/bench_luby.json 2> gpurun_out/bench_luby.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -k regex:"k_|gc" --csv --log-file gpurun_out/launches_count.csv python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/ncu_bench.log 2>&1
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:k_count_persistent -c 1 -o gpurun_out/prof_count_persistent5 python tools/ncu_one.py --mode count > gpurun_out/ncu_full6.log 2>&1
timeout 900 python tools/bench_configs.py > gpurun_out/configs.jsonl 2> gpurun_out/configs.err
timeout 300 python tools/round_profile.py --scale 24 --mode count --out gpurun_out/rounds_count.json > gpurun_out/rounds_count.log 2>&1
timeout 600 python tools/dbg/count_variants.py > gpurun_out/mhl.jsonl 2>&1 || true
