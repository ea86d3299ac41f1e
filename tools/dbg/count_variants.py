"""R-MAT s24 / mesh: every variant in COUNT mode (one JSON line each)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import graphgen as G  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402
import tools.bench_configs as B  # noqa: E402

g4 = G.config_graph("cfg4", "cuda")
for H in (2, 4, 8):
    B.run("cfg4 R-MAT s24", g4, gcb.MULTIHASH(H), f"multihash H={H}", "count")
B.run("cfg4 R-MAT s24", g4, gcb.LUBY_MIS, "luby", "count")
B.run("cfg4 R-MAT s24", g4, gcb.IS_ALG2, "is_alg2", "count")
B.run("cfg4 R-MAT s24", g4, gcb.JP_ALG4, "jp_alg4", "count")
del g4
g3 = G.config_graph("cfg3", "cuda")
B.run("cfg3 mesh 128^3", g3, gcb.MAXMIN, "maxmin", "count")
B.run("cfg3 mesh 128^3", g3, gcb.MULTIHASH(4), "multihash H=4", "count")
