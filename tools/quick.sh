# Quick GPU check of the COUNT path: max-min parity subset + a short bench line.
# usage (on the GPU box): bash tools/quick.sh TAG
T=${1:-q}
python -m pytest tests/test_gpu_parity.py -x -q -k "golden or random_small or adversarial or duplicates or cfg1 or cfg2 or s18 or cfg4_rmat_s24_certificate or ldf_random or rgg" > gpurun_out/${T}_pytest.log 2>&1; tail -2 gpurun_out/${T}_pytest.log
python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err
python -c "
import json;d=json.loads(open('gpurun_out/${T}_bench.json').read().strip().splitlines()[-1])
c=d['roofline']['classes']
print('ms', round(d['ms_per_step'],3), 'GTEPS', round(d['value'],2), {k:round(v['launch_ms_median'],3) for k,v in c.items()}, 'colours', d.get('n_colors'), 'rounds', d.get('rounds'))"
