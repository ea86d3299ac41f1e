timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q -m gpu > gpurun_out/pt_rw.log 2>&1; echo rc=$? >> gpurun_out/pt_rw.log
bash tools/dbg/ab.sh libgc_head.so > gpurun_out/ab_rw.txt 2>&1
