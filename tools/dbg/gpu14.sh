timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "golden or random or adversarial or s18 or s24 or cfg2 or cfg1" > gpurun_out/pt_rd.log 2>&1; echo rc=$? >> gpurun_out/pt_rd.log
bash tools/dbg/ab.sh libgc_prev.so > gpurun_out/ab_rd.txt 2>&1
