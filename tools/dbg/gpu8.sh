timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "golden or random or adversarial or s18 or s24 or cfg2 or cfg3 or dupl" > gpurun_out/pt_skip.log 2>&1; echo rc=$? >> gpurun_out/pt_skip.log
bash tools/dbg/ab.sh libgc_noskip.so > gpurun_out/ab_skip.txt 2>&1
