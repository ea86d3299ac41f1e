timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node=1 --master-addr=127.0.0.1 --master-port=29512 bench.py --dist --steps 3 --warmup 3 --no-cpu-baseline > gpurun_out/bench_dist_s24.log 2>&1; echo rc=$? >> gpurun_out/bench_dist_s24.log
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "s25" > gpurun_out/pt_s25.log 2>&1; echo rc=$? >> gpurun_out/pt_s25.log
