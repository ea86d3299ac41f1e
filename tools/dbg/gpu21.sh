timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q -m gpu > gpurun_out/pt_gc.log 2>&1; echo rc=$? >> gpurun_out/pt_gc.log
bash tools/dbg/ab.sh libgc_nogc256.so > gpurun_out/ab_gc1.txt 2>&1
bash tools/dbg/ab.sh libgc_gc1024.so > gpurun_out/ab_gc2.txt 2>&1
cat > /tmp/mhl.py <<'PY'
import sys; sys.path.insert(0, '.')
import tools.bench_configs as B, graphgen as G, paper_conf_ipps_osamatybo19_b200 as gcb
g4 = G.config_graph("cfg4", "cuda")
for H in (2, 4, 8):
    B.run("cfg4 R-MAT s24", g4, gcb.MULTIHASH(H), f"multihash H={H}", "count")
B.run("cfg4 R-MAT s24", g4, gcb.LUBY_MIS, "luby", "count")
B.run("cfg4 R-MAT s24", g4, gcb.IS_ALG2, "is_alg2", "count")
B.run("cfg4 R-MAT s24", g4, gcb.JP_ALG4, "jp_alg4", "count")
g3 = G.config_graph("cfg3", "cuda")
B.run("cfg3 mesh 128^3", g3, gcb.MAXMIN, "maxmin", "count")
B.run("cfg3 mesh 128^3", g3, gcb.MULTIHASH(4), "multihash H=4", "count")
PY
timeout 600 python /tmp/mhl.py > gpurun_out/mhl.jsonl 2>&1
