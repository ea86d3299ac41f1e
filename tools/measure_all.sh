set -x
python -m pytest tests -m gpu -x -q > gpurun_out/m_pytest.log 2>&1; tail -2 gpurun_out/m_pytest.log
python bench.py --steps 10 --warmup 3 > gpurun_out/m_bench.json 2> gpurun_out/m_bench.err
ncu --metrics gpu__time_duration.sum --clock-control none -k regex:"k_|fill" --csv --log-file gpurun_out/m_launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_count -c 3 -o gpurun_out/m_prof python tools/count_blocks_sweep.py 24 > gpurun_out/m_ncu.log 2>&1
ls -la gpurun_out
