# A/B of library variants on the partitioned COUNT rounds (loopback, R-MAT s22).
for L in "$@"; do
  if [ "$L" = "-" ]; then unset GC_LIB_PATH; else export GC_LIB_PATH=$L; fi
  echo "$L"; python tools/loopback_timing.py 22 2>/dev/null | cut -c1-120
done
