timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "loopback" > gpurun_out/pt_dist.log 2>&1; echo rc=$? >> gpurun_out/pt_dist.log
cat > /tmp/lb.py <<'PY'
import sys; sys.path.insert(0, '.')
import tools.bench_configs as B, graphgen as G, paper_conf_ipps_osamatybo19_b200 as gcb
g5 = G.rmat(22, 16, seed=1, device="cuda")
for p in (1, 2, 4, 8):
    B.run("R-MAT s22 partitioned", g5, gcb.MAXMIN, "maxmin", mode="auto", reps=2, warm=1, loopback=p)
B.run("R-MAT s22", g5, gcb.MAXMIN, "maxmin", mode="count", reps=2, warm=1)
PY
timeout 600 python /tmp/lb.py > gpurun_out/lb.jsonl 2>&1
