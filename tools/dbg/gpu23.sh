bash tools/dbg/ab.sh libgc_t640.so > gpurun_out/ab_t640.txt 2>&1
bash tools/dbg/ab.sh libgc_t768.so > gpurun_out/ab_t768.txt 2>&1
bash tools/dbg/ab.sh libgc_t384.so > gpurun_out/ab_t384.txt 2>&1
