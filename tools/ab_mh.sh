# A/B timing of library variants on R-MAT s24 multi-hash H (COUNT).
T=$1; H=$2; shift; shift
for rep in 1 2; do
for L in "$@"; do
  if [ "$L" = "-" ]; then unset GC_LIB_PATH; else export GC_LIB_PATH=$L; fi
  python bench.py --steps 3 --warmup 3 --variant multihash --hashes $H --mode count --no-e2e --no-cpu-baseline --no-profile > gpurun_out/${T}_abm.json 2>/dev/null
  python -c "
import json;d=json.loads(open('gpurun_out/${T}_abm.json').read().strip().splitlines()[-1])
print('$L', 'mh H=$H ms', round(d['ms_per_step'],3), d.get('n_colors'), d.get('rounds'))"
done; done
