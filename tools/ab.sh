# A/B timing of library variants on R-MAT s24 max-min (bench.py, kernel-only line).
# usage: bash tools/ab.sh TAG lib1 lib2 ...   (a lib of "-" = the in-tree libgc.so)
T=$1; shift
for rep in 1 2; do
for L in "$@"; do
  if [ "$L" = "-" ]; then unset GC_LIB_PATH; else export GC_LIB_PATH=$L; fi
  python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/${T}_ab.json 2>/dev/null
  python -c "
import json;d=json.loads(open('gpurun_out/${T}_ab.json').read().strip().splitlines()[-1])
c=d['roofline']['classes']
print('$L', 'ms', round(d['ms_per_step'],3), {k:round(v['launch_ms_median'],3) for k,v in c.items()}, d.get('n_colors'), d.get('rounds'))"
done; done
