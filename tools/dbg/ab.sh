# A/B: default libgc.so vs tools/dbg/lib/$1 (bench only, 3 alternating runs each)
for i in 1 2 3; do
  timeout 300 python bench.py --mode count --no-cpu-baseline --no-e2e --no-profile 2>/dev/null | python -c "import json,sys; print('A', json.load(sys.stdin)['ms_per_step'])"
  GC_LIB_PATH=tools/dbg/lib/$1 timeout 300 python bench.py --mode count --no-cpu-baseline --no-e2e --no-profile 2>/dev/null | python -c "import json,sys; print('B', json.load(sys.stdin)['ms_per_step'])"
done
