timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q -m gpu > gpurun_out/pt_st.log 2>&1; echo rc=$? >> gpurun_out/pt_st.log
bash tools/dbg/ab.sh libgc_prejpv.so > gpurun_out/ab_st1.txt 2>&1
bash tools/dbg/ab.sh libgc_st2048.so > gpurun_out/ab_st2.txt 2>&1
