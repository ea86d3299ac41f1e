timeout 1200 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "golden or random or adversarial or alg2" > gpurun_out/pt_n3.log 2>&1; echo rc=$? >> gpurun_out/pt_n3.log
cat > /tmp/n3.py <<'PY'
import sys; sys.path.insert(0, '.')
import tools.bench_configs as B, graphgen as G, paper_conf_ipps_osamatybo19_b200 as gcb
g4 = G.config_graph("cfg4", "cuda")
B.run("cfg4 R-MAT s24", g4, gcb.IS_ALG2, "is_alg2 (max-only)", "count")
B.run("cfg4 R-MAT s24", g4, gcb.JP_ALG4, "jp_alg4 (GraphBLAS JP)", "count")
B.run("cfg4 R-MAT s24", g4, gcb.LUBY_MIS, "luby", "count")
B.run("cfg4 R-MAT s24", g4, gcb.MAXMIN, "maxmin", "count")
g2 = G.config_graph("cfg2", "cuda")
for v, nm in ((gcb.IS_ALG2, "is_alg2"), (gcb.JP_ALG4, "jp_alg4"), (gcb.LUBY_MIS, "luby"), (gcb.MAXMIN, "maxmin")):
    B.run("cfg2 ER 2^20 d16", g2, v, nm, "count")
PY
timeout 600 python /tmp/n3.py > gpurun_out/n3.jsonl 2>&1
