# Round-end measurement pass on one B200 (gpurun): tests, bench line, ncu
# launch list and full capture, configuration sweeps.  Outputs in gpurun_out/.
set -x
python -m pytest tests -m gpu -x -q > gpurun_out/m_pytest.log 2>&1; tail -2 gpurun_out/m_pytest.log
python bench.py --steps 10 --warmup 3 > gpurun_out/m_bench.json 2> gpurun_out/m_bench.err
python bench.py --steps 5 --warmup 3 --variant luby --no-e2e --no-cpu-baseline > gpurun_out/m_bench_luby.json 2>/dev/null
ncu --metrics gpu__time_duration.sum --clock-control none -k regex:"k_|fill" --csv --log-file gpurun_out/m_launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_count -c 3 -o gpurun_out/m_prof python tools/count_blocks_sweep.py 24 > gpurun_out/m_ncu.log 2>&1
python tools/bench_configs.py > gpurun_out/m_configs.jsonl 2> gpurun_out/m_configs.err
python tools/rgg_sweep.py > gpurun_out/m_rgg_sweep.jsonl 2> gpurun_out/m_rgg.err
python tools/table2.py > gpurun_out/m_table2.jsonl 2> gpurun_out/m_table2.err
python tools/ldf_compare.py > gpurun_out/m_ldf.jsonl 2> gpurun_out/m_ldf.err
python tools/loopback_timing.py 22 > gpurun_out/m_loopback.jsonl 2> gpurun_out/m_loopback.err
ls -la gpurun_out
