# A/B timing of library variants on R-MAT s24 Luby (JP COUNT).
T=$1; shift
for rep in 1 2; do
for L in "$@"; do
  if [ "$L" = "-" ]; then unset GC_LIB_PATH; else export GC_LIB_PATH=$L; fi
  python bench.py --steps 5 --warmup 3 --variant luby --no-e2e --no-cpu-baseline > gpurun_out/${T}_abl.json 2>/dev/null
  python -c "
import json;d=json.loads(open('gpurun_out/${T}_abl.json').read().strip().splitlines()[-1])
print('$L', 'luby ms', round(d['ms_per_step'],3), d.get('n_colors'), d.get('rounds'))"
done; done
