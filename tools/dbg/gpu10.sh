timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "not loopback" > gpurun_out/pt_stream.log 2>&1; echo rc=$? >> gpurun_out/pt_stream.log
bash tools/dbg/ab.sh libgc_nostream.so > gpurun_out/ab_stream.txt 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_count" --csv --log-file gpurun_out/launches_stream.csv python tools/ncu_one.py --mode count > gpurun_out/ncu_stream.log 2>&1
