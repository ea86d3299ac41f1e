timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q -m gpu > gpurun_out/pt_st.log 2>&1; echo rc=$? >> gpurun_out/pt_st.log
bash tools/dbg/ab.sh libgc_st512.so > gpurun_out/ab_st512.txt 2>&1
bash tools/dbg/ab.sh libgc_st256.so > gpurun_out/ab_st256.txt 2>&1
