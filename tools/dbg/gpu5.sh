timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "multihash or golden or random or adversarial" > gpurun_out/pt_mh2.log 2>&1; echo rc=$? >> gpurun_out/pt_mh2.log
cat > /tmp/mh.py <<'PY'
import sys; sys.path.insert(0, '.')
import tools.bench_configs as B, graphgen as G, paper_conf_ipps_osamatybo19_b200 as gcb
g4 = G.config_graph("cfg4", "cuda")
for H in (2, 4, 8, 16):
    B.run("cfg4 R-MAT s24", g4, gcb.MULTIHASH(H), f"multihash H={H}", "count")
PY
timeout 300 python /tmp/mh.py > gpurun_out/mh.jsonl 2>&1
