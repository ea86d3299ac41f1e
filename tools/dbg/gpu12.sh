timeout 300 python -m pytest tests/test_gpu_nccl.py -v -m gpu > gpurun_out/pt_nccl.log 2>&1; echo rc=$? >> gpurun_out/pt_nccl.log
timeout 300 python -m torch.distributed.run --nnodes=1 --nproc-per-node=1 --master-addr=127.0.0.1 --master-port=29511 bench.py --dist --scale 16 --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/bench_dist_s16.log 2>&1; echo rc=$? >> gpurun_out/bench_dist_s16.log
