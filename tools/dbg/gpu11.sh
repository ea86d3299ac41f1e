timeout 1500 python -m pytest tests/ -x -q -m gpu > gpurun_out/pt_all.log 2>&1; echo rc=$? >> gpurun_out/pt_all.log
bash tools/dbg/ab.sh libgc_nostream.so > gpurun_out/ab_stream2.txt 2>&1
timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node=1 --master-addr=127.0.0.1 --master-port=29511 bench.py --dist --steps 5 --warmup 3 > gpurun_out/bench_dist1.json 2> gpurun_out/bench_dist1.err
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_count_stream" --csv --log-file gpurun_out/launches_stream2.csv python tools/ncu_one.py --mode count > gpurun_out/ncu_stream2.log 2>&1
