"""Decrements of the COUNT rounds on R-MAT s<scale>, computed from the ORACLE's
colouring (no GPU): entries, decrements left after the dead-side skip, and
how many of those still reach an uncoloured vertex; per-round atomics and the
largest number of decrements one count word receives in a round.

    python tools/dead_atomics.py 22
"""
import os, sys, time, numpy as np
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import graphgen as G, oracle as O
s = int(sys.argv[1])
t=time.time(); g = G.rmat(s, 16, seed=1); print('gen', time.time()-t, g.n, g.nnz, flush=True)
t=time.time(); C = O.color_maxmin(g, 1).astype(np.int64); print('oracle', time.time()-t, flush=True)
ro = g.row_offsets.numpy(); ci = g.col_indices.numpy().astype(np.int64)
n = g.n
R = C >> 1                       # round of each vertex
p = O.priorities(1, 0, n).astype(np.int64)
deg = np.diff(ro)
src = np.repeat(np.arange(n), deg)
dst = ci
# v = src walks (in round R[src]); side: v larger than w -> decrements hi(w)
vlarger = p[src] > p[dst]
# scheduling side of v: lo side free first? colour odd = min colour... use: lo side free at start
# of round R[v] <=> all smaller neighbours coloured before; approximate with colour parity (odd = lo free)
lofree = (C[src] & 1) == 1
dead = np.where(lofree, vlarger, ~vlarger)          # skipped entries
live = ~dead
print('entries', len(dst), 'live', live.sum(), 'useful(dst uncoloured after)', (R[dst] > R[src]).sum())
r = R[src][live]; d = dst[live]
key = r * n + d
u, cnt = np.unique(key, return_counts=True)
rr = u // n
mx = np.zeros(R.max() + 1, np.int64); np.maximum.at(mx, rr, cnt)
tot = np.bincount(r, minlength=R.max() + 1)
for lo, hi in [(0,1),(1,10),(10,100),(100,1000),(1000,2000),(2000,R.max()+1)]:
    if lo > R.max(): break
    print(lo, hi, 'atomics/round', int(tot[lo:hi].mean()), 'max same-address/round', int(mx[lo:hi].mean()), 'max', int(mx[lo:hi].max()))

# decrements to vertices coloured earlier than the walker, by the target's round
# (what a residual-row compaction after round K would remove)
rv = R[src][live]; rw = R[dst][live]
dead_mask = rw < rv
print('issued', live.sum(), 'to coloured targets', dead_mask.sum())
for K in [1, 2, 3, 5, 10, 50]:
    # compaction at the start of round K removes entries to vertices coloured in rounds < K
    # from the rows walked in rounds >= K
    rem = (dead_mask & (rw < K) & (rv >= K)).sum()
    rows_after = (R >= K)
    ent_after = deg[rows_after].sum()
    print(f'compact at round {K}: removes {rem} issued decrements; rows left {rows_after.sum()}, their entries {ent_after}')
