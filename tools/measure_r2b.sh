# Round-2 measurement pass on one B200 (gpurun): tests, smoke, bench lines, ncu
# launch list and full capture of the COUNT kernels, configuration sweeps.
T=${1:-m2}
python -m pytest tests -m gpu -x -q > gpurun_out/${T}_pytest.log 2>&1; tail -2 gpurun_out/${T}_pytest.log
python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${T}_smoke.log 2>&1; tail -1 gpurun_out/${T}_smoke.log
python bench.py --steps 10 --warmup 3 > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err
python bench.py --steps 5 --warmup 3 --variant luby --no-e2e --no-cpu-baseline > gpurun_out/${T}_bench_luby.json 2>/dev/null
ncu --metrics gpu__time_duration.sum --clock-control none -k regex:"k_|fill" --csv --log-file gpurun_out/${T}_launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:"k_count_persistent|k_count_warp|k_count_zero" -c 3 -o gpurun_out/${T}_prof python tools/ncu_one.py --mode count > gpurun_out/${T}_ncu.log 2>&1
python tools/round_profile.py --scale 24 --mode count --out gpurun_out/${T}_rounds.json > /dev/null 2>&1
timeout 600 python tools/bench_configs.py > gpurun_out/${T}_configs.jsonl 2> gpurun_out/${T}_configs.err
timeout 600 python tools/rgg_sweep.py > gpurun_out/${T}_rgg_sweep.jsonl 2> gpurun_out/${T}_rgg.err
ls gpurun_out | grep ${T}_
