timeout 600 python tools/dbg/n3dbg.py > gpurun_out/n3dbg.log 2>&1
bash tools/dbg/ab.sh libgc_prejpv.so > gpurun_out/ab_n3.txt 2>&1
