# Duration of k_count_persistent stopped after R rounds (GC_MAX_ROUNDS=R; 0 = the init phase only),
# ncu launch times of the second colouring of R-MAT s24: init, round 0, round 1 by difference.
for R in 0 1 2 3; do
  GC_MAX_ROUNDS=$R ncu --metrics gpu__time_duration.sum --clock-control none -k regex:k_count_persistent --csv \
     --log-file gpurun_out/ph_$R.csv python tools/ncu_one.py --mode count --warm > /dev/null 2>&1
  echo "R=$R $(grep k_count_persistent gpurun_out/ph_$R.csv | tail -1 | awk -F'","' '{print $NF}')"
done
