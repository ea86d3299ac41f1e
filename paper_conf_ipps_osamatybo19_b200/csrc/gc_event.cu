// gc_event.cu -- EVENT mode of the max-min colouring (H = 1): the same rounds
// and the same colours as Alg.5, computed work-efficiently.
//
// Why: on power-law graphs the round count reaches thousands (R-MAT s24:
// 2,518 rounds) while most uncoloured vertices stay blocked for hundreds of
// rounds.  The paper's ComputeOp re-scans every uncoloured row every round
// (its "serial for loop" flaw); measured on B200 the
// sweep mode visits ~335 x nnz entries per colouring at s24.
//
// How: v is blocked in round k iff it has an
// uncoloured neighbour with a larger weight (a "hi witness") and one with a
// smaller weight (a "lo witness") -- Alg.5 L29-34 leave both colormax and
// colormin false.  Each blocked vertex keeps one witness per side, W[v], and
// the row position of each, P[v], chosen as the FIRST qualifying neighbour at
// or after a cursor.  Weights are fixed and colouring is monotone, so every
// row entry before the witness is either coloured or on the other side, now
// and forever; when a witness is coloured the search resumes right after it.
// v's outcome can only change when one of its witnesses is coloured, so a
// round evaluates only the vertices whose witness was coloured in the
// previous round (found by walking the rows of newly coloured vertices).
// Each side's cursor only moves forward: the whole colouring reads each row
// O(1) times instead of once per round.
//
// Round k: k_eval (vertices of D_k; lane / warp scans) -> k_eval_big (CTA per
// long remaining scan) -> k_notify (rows of the vertices coloured in round k;
// lane / warp) -> k_notify_big (rows of long coloured vertices split across
// the whole grid).  Status test: u is uncoloured at the start of round k iff
// C[u] >= 2k (as in sweep mode), so in-place colour writes are race-free.
#include "gc_event_common.cuh"

namespace gc {

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st);
int ensure_nk(gc_graph *g, int64_t need);

namespace {

using namespace ev;
constexpr int kBlock = 256;
constexpr int kBigBlock = 512;
constexpr int kSeg = 128;  // entries per long-row notify item (4 per lane)

// counter slots in g->s.ctr used by this mode
enum : int {
    kD = 24,      // [24..26] |D_k| rotating k % 3
    kI = 27,      // [27..29] |I_k| (coloured in round k)
    kBE = 30,     // [30..32] long-scan queue of round k
    kBN = 33,     // [33..35] long-row notify queue of round k
    kRem = 36,    // uncoloured vertices
    kVisE = 37,   // PROF: entries scanned by k_eval
    kVisB = 38,   // PROF: entries scanned by k_eval_big
    kVisN = 39,   // PROF: entries walked by the notify kernels
    kSumD = 40    // PROF: sum of |D_k|
};

template <bool PROF>
__global__ void __launch_bounds__(kBlock) k_eval(
    const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci, uint32_t *C, uint2 *W,
    uint2 *P, const uint32_t *__restrict__ Din, uint32_t *__restrict__ Iout,
    uint32_t *__restrict__ bigq, unsigned long long *ctr, int64_t *nk, int64_t *rstat,
    int64_t nk_cap, uint32_t k, uint32_t key, int dense, int64_t n, uint32_t thread_max,
    uint32_t big_min) {
    const unsigned long long N = dense ? (unsigned long long)n : ctr[kD + k % 3];
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        ctr[kD + (k + 2) % 3] = 0;
        ctr[kI + (k + 1) % 3] = 0;
        ctr[kBE + (k + 1) % 3] = 0;
        ctr[kBN + k % 3] = 0;
        if ((int64_t)k < nk_cap) nk[k] = (int64_t)ctr[kRem];
        if (PROF) {
            ctr[kSumD] += N;
            if ((int64_t)k < nk_cap) rstat[16 * k] = (int64_t)N;
        }
    }
    const uint32_t thresh = 2u * k;
    const unsigned lane = lane_id();
    const unsigned long long nwarps = ((unsigned long long)gridDim.x * blockDim.x) >> 5;
    const unsigned long long warp0 = ((unsigned long long)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    if (!dense && N <= nwarps) {
        // few vertices (the common late round): one warp per vertex, so the
        // scans of different vertices run in parallel instead of in one warp
        if (warp0 < N) {
            const uint32_t v = Din[warp0];
            const int64_t rs = ro[v], re = ro[v + 1];
            const Resume r = resume_of(v, rs, false, W, P, C, thresh);
            int64_t s = r.need_hi ? r.sh : re;
            if (r.need_lo && r.sl < s) s = r.sl;
            const bool work = r.need_hi || r.need_lo;
            const bool big = work && re - s >= (int64_t)big_min;
            uint32_t nvis = 0;
            if (work && !big) {
                Found f;
                warp_search(ci, C, thresh, key, weight_mix(v ^ key), r.need_hi, r.need_lo, r.sh,
                            r.sl, re, f, nvis);
                if (lane == 0 && settle(v, rs, r, f, k, C, W, P))
                    Iout[atomicAdd(&ctr[kI + k % 3], 1ull)] = v;
            }
            if (big && lane == 0) bigq[atomicAdd(&ctr[kBE + k % 3], 1ull)] = v;
            if (PROF) {
                const unsigned tot = __reduce_add_sync(kFull, nvis);
                if (lane == 0 && tot) atomicAdd(&ctr[kVisE], (unsigned long long)tot);
            }
        }
        return;
    }
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (unsigned long long base = (unsigned long long)blockIdx.x * blockDim.x + (threadIdx.x & ~31u);
         base < N; base += stride) {
        const unsigned long long idx = base + lane;
        const bool valid = idx < N;
        uint32_t v = 0;
        int64_t rs = 0, re = 0;
        Resume r{false, false, 0, 0};
        if (valid) {
            v = dense ? (uint32_t)idx : Din[idx];
            rs = ro[v];
            re = ro[v + 1];
            r = resume_of(v, rs, dense != 0, W, P, C, thresh);
        }
        const bool work = valid && (r.need_hi || r.need_lo);
        int64_t s = r.need_hi ? r.sh : re;
        if (r.need_lo && r.sl < s) s = r.sl;
        const int64_t remaining = re - s;
        const bool small = work && remaining <= (int64_t)thread_max;
        const bool big = work && !small && remaining >= (int64_t)big_min;
        const bool mid = work && !small && !big;
        const uint32_t pv = weight_mix(v ^ key);
        Found f;
        uint32_t nvis = 0;
        if (small) lane_search(ci, C, thresh, key, pv, r.need_hi, r.need_lo, r.sh, r.sl, re, f, nvis);
        unsigned mm = __ballot_sync(kFull, mid);
        while (mm) {
            const int src = __ffs(mm) - 1;
            mm &= mm - 1;
            const uint32_t pw = __shfl_sync(kFull, pv, src);
            const bool nh = __shfl_sync(kFull, r.need_hi, src);
            const bool nl = __shfl_sync(kFull, r.need_lo, src);
            const int64_t sh = __shfl_sync(kFull, r.sh, src);
            const int64_t sl = __shfl_sync(kFull, r.sl, src);
            const int64_t we = __shfl_sync(kFull, re, src);
            Found fw;
            uint32_t wv = 0;
            warp_search(ci, C, thresh, key, pw, nh, nl, sh, sl, we, fw, wv);
            if ((int)lane == src) f = fw;
            if (PROF) nvis += wv;
        }
        bool colored = false;
        if (small || mid) colored = settle(v, rs, r, f, k, C, W, P);
        warp_append(colored, v, Iout, &ctr[kI + k % 3]);
        warp_append(big, v, bigq, &ctr[kBE + k % 3]);
        if (PROF) {
            const unsigned tot = __reduce_add_sync(kFull, nvis);
            if (lane == 0 && tot) atomicAdd(&ctr[kVisE], (unsigned long long)tot);
        }
    }
}

// CTA per long remaining scan, early exit per 2048-entry chunk.
template <bool PROF>
__global__ void __launch_bounds__(kBigBlock) k_eval_big(
    const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci, uint32_t *C, uint2 *W,
    uint2 *P, const uint32_t *__restrict__ bigq, uint32_t *__restrict__ Iout,
    unsigned long long *ctr, uint32_t k, uint32_t key, int dense) {
    const unsigned long long nbig = ctr[kBE + k % 3];
    const uint32_t thresh = 2u * k;
    __shared__ unsigned long long sh_h, sh_l;  // min absolute position found
    constexpr int kUnroll = 4;
    uint32_t nvis = 0;
    for (unsigned long long i = blockIdx.x; i < nbig; i += gridDim.x) {
        const uint32_t v = bigq[i];
        const int64_t rs = ro[v], re = ro[v + 1];
        const Resume r = resume_of(v, rs, dense != 0, W, P, C, thresh);
        const uint32_t pv = weight_mix(v ^ key);
        if (threadIdx.x == 0) {
            sh_h = ~0ull;
            sh_l = ~0ull;
        }
        __syncthreads();
        int64_t s = r.need_hi ? r.sh : re;
        if (r.need_lo && r.sl < s) s = r.sl;
        unsigned long long H = ~0ull, L = ~0ull;
        for (int64_t e0 = s; e0 < re; e0 += (int64_t)blockDim.x * kUnroll) {
            uint32_t u[kUnroll], c[kUnroll];
#pragma unroll
            for (int q = 0; q < kUnroll; ++q) {
                const int64_t e = e0 + threadIdx.x + (int64_t)q * blockDim.x;
                u[q] = e < re ? ci[e] : 0u;
            }
#pragma unroll
            for (int q = 0; q < kUnroll; ++q) {
                const int64_t e = e0 + threadIdx.x + (int64_t)q * blockDim.x;
                c[q] = e < re ? C[u[q]] : 0u;
            }
            uint32_t rh = 0xFFFFFFFFu, rl = 0xFFFFFFFFu;  // first hit, relative to e0
#pragma unroll
            for (int q = 0; q < kUnroll; ++q) {
                const int64_t e = e0 + threadIdx.x + (int64_t)q * blockDim.x;
                if (PROF) nvis += e < re;
                if (e < re && c[q] >= thresh) {
                    const uint32_t pu = weight_mix(u[q] ^ key);
                    const uint32_t rel = (uint32_t)(e - e0);
                    if (r.need_hi && e >= r.sh && pu > pv) rh = min(rh, rel);
                    if (r.need_lo && e >= r.sl && pu < pv) rl = min(rl, rel);
                }
            }
            rh = __reduce_min_sync(kFull, rh);
            rl = __reduce_min_sync(kFull, rl);
            const unsigned long long mh = rh == 0xFFFFFFFFu ? ~0ull : (unsigned long long)(e0 + rh);
            const unsigned long long ml = rl == 0xFFFFFFFFu ? ~0ull : (unsigned long long)(e0 + rl);
            if ((threadIdx.x & 31) == 0) {
                if (mh != ~0ull) atomicMin(&sh_h, mh);
                if (ml != ~0ull) atomicMin(&sh_l, ml);
            }
            __syncthreads();
            H = sh_h;
            L = sh_l;
            __syncthreads();
            if ((!r.need_hi || H != ~0ull) && (!r.need_lo || L != ~0ull)) break;
        }
        if (threadIdx.x == 0) {
            Found f;
            if (H != ~0ull) {
                f.hpos = (int64_t)H;
                f.hw = ci[H];
            }
            if (L != ~0ull) {
                f.lpos = (int64_t)L;
                f.lw = ci[L];
            }
            if (settle(v, rs, r, f, k, C, W, P)) {
                const unsigned long long pos = atomicAdd(&ctr[kI + k % 3], 1ull);
                Iout[pos] = v;
            }
        }
        __syncthreads();
    }
    if (PROF) {
        const unsigned tot = __reduce_add_sync(kFull, nvis);
        if ((threadIdx.x & 31) == 0 && tot) atomicAdd(&ctr[kVisB], (unsigned long long)tot);
    }
}

template <bool PROF>
__global__ void __launch_bounds__(kBlock) k_notify(
    const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci, const uint32_t *C,
    const uint2 *W, uint32_t *S, const uint32_t *__restrict__ Iin, uint32_t *__restrict__ Dout,
    uint2 *__restrict__ bigq, unsigned long long *ctr, uint32_t k, uint32_t thread_max,
    uint32_t big_min) {
    const unsigned long long cnt = ctr[kI + k % 3];
    if (blockIdx.x == 0 && threadIdx.x == 0) ctr[kRem] -= cnt;
    unsigned long long *dcount = &ctr[kD + (k + 1) % 3];
    const unsigned lane = lane_id();
    uint32_t nvis = 0;
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (unsigned long long base = (unsigned long long)blockIdx.x * blockDim.x + (threadIdx.x & ~31u);
         base < cnt; base += stride) {
        const unsigned long long idx = base + lane;
        const bool valid = idx < cnt;
        uint32_t u = 0;
        int64_t rs = 0, re = 0;
        if (valid) {
            u = Iin[idx];
            rs = ro[u];
            re = ro[u + 1];
        }
        const int64_t deg = re - rs;
        const bool small = valid && deg <= (int64_t)thread_max;
        const bool big = valid && !small;
        if (small) {
            for (int64_t e = rs; e < re; ++e) {
                const uint32_t w = ci[e];
                if (wake(w, u, k, C, W, S)) Dout[atomicAdd(dcount, 1ull)] = w;
            }
            if (PROF) nvis += (uint32_t)deg;
        }
        // long rows: one work item per kSeg-entry segment, spread over the grid
        unsigned bm = __ballot_sync(kFull, big);
        while (bm) {
            const int src = __ffs(bm) - 1;
            bm &= bm - 1;
            const uint32_t uu = __shfl_sync(kFull, u, src);
            const int64_t dg = __shfl_sync(kFull, deg, src);
            const uint32_t nseg = (uint32_t)((dg + kSeg - 1) / kSeg);
            unsigned long long b0 = 0;
            if (lane == 0) b0 = atomicAdd(&ctr[kBN + k % 3], (unsigned long long)nseg);
            b0 = __shfl_sync(kFull, b0, 0);
            for (uint32_t q = lane; q < nseg; q += 32) bigq[b0 + q] = make_uint2(uu, q);
        }
    }
    if (PROF) {
        const unsigned tot = __reduce_add_sync(kFull, nvis);
        if (lane == 0 && tot) atomicAdd(&ctr[kVisN], (unsigned long long)tot);
    }
}

// Segments of long coloured rows: one warp per kSeg-entry segment.
template <bool PROF>
__global__ void __launch_bounds__(kBlock) k_notify_big(
    const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci, const uint32_t *C,
    const uint2 *W, uint32_t *S, const uint2 *__restrict__ bigq, uint32_t *__restrict__ Dout,
    unsigned long long *ctr, uint32_t k, int64_t *rstat, int64_t nk_cap) {
    const unsigned long long nitems = ctr[kBN + k % 3];
    unsigned long long *dcount = &ctr[kD + (k + 1) % 3];
    if (PROF && blockIdx.x == 0 && threadIdx.x == 0 && (int64_t)k < nk_cap) {
        rstat[16 * k + 1] = (int64_t)ctr[kI + k % 3];
        rstat[16 * k + 2] = (int64_t)ctr[kBE + k % 3];
        rstat[16 * k + 3] = (int64_t)nitems;
    }
    const unsigned lane = lane_id();
    uint32_t nvis = 0;
    const unsigned long long warp0 = ((unsigned long long)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const unsigned long long nwarps = ((unsigned long long)gridDim.x * blockDim.x) >> 5;
    for (unsigned long long it = warp0; it < nitems; it += nwarps) {
        const uint2 item = bigq[it];
        const uint32_t u = item.x;
        const int64_t rs = ro[u] + (int64_t)item.y * kSeg;
        const int64_t re = min(ro[u + 1], rs + (int64_t)kSeg);
        uint32_t w[kSeg / 32];
#pragma unroll
        for (int q = 0; q < kSeg / 32; ++q) {
            const int64_t e = rs + q * 32 + lane;
            w[q] = e < re ? ci[e] : 0xFFFFFFFFu;
        }
#pragma unroll
        for (int q = 0; q < kSeg / 32; ++q) {
            const bool wk = w[q] != 0xFFFFFFFFu && wake(w[q], u, k, C, W, S);
            warp_append(wk, w[q], Dout, dcount);
        }
        if (PROF && lane == 0) nvis += (uint32_t)(re - rs);
    }
    if (PROF) {
        const unsigned tot = __reduce_add_sync(kFull, nvis);
        if (lane == 0 && tot) atomicAdd(&ctr[kVisN], (unsigned long long)tot);
    }
}

template <bool PROF>
int launch_round(gc_graph *g, const RunParams &p, uint32_t k, int grid, int grid_dense,
                 EventTimer *tm) {
    Scratch &s = g->s;
    uint2 *W = reinterpret_cast<uint2 *>(s.W);
    uint2 *P = reinterpret_cast<uint2 *>(s.P);
    const uint32_t key = p.keys.k[0];
    const int dense = k == 0 ? 1 : 0;
    uint32_t *D[2] = {s.F[0], s.F[1]};
    uint32_t *I = s.hub;
    int rc;
    if (PROF && (rc = tm->begin(g->stream, 0))) return rc;
    k_eval<PROF><<<dense ? grid_dense : grid, kBlock, 0, g->stream>>>(
        g->ro, g->ci, s.C, W, P, D[k % 2], I, s.Q, s.ctr, s.nk, s.rstat, s.nk_cap, k, key, dense,
        g->n,
        (uint32_t)p.thread_deg_max, (uint32_t)p.eval_big_min);
    if (PROF && (rc = tm->end(g->stream))) return rc;
    if (PROF && (rc = tm->begin(g->stream, 1))) return rc;
    k_eval_big<PROF><<<g->sm_count * 2, kBigBlock, 0, g->stream>>>(g->ro, g->ci, s.C, W, P, s.Q, I,
                                                                   s.ctr, k, key, dense);
    if (PROF && (rc = tm->end(g->stream))) return rc;
    if (PROF && (rc = tm->begin(g->stream, 2))) return rc;
    uint2 *Q2 = reinterpret_cast<uint2 *>(s.Q2);
    k_notify<PROF><<<grid, kBlock, 0, g->stream>>>(g->ro, g->ci, s.C, W, s.S, I, D[(k + 1) % 2],
                                                   Q2, s.ctr, k, (uint32_t)p.thread_deg_max, 0u);
    if (PROF && (rc = tm->end(g->stream))) return rc;
    if (PROF && (rc = tm->begin(g->stream, 3))) return rc;
    k_notify_big<PROF><<<g->sm_count * 8, kBlock, 0, g->stream>>>(g->ro, g->ci, s.C, W, s.S, Q2,
                                                                  D[(k + 1) % 2], s.ctr, k,
                                                                  s.rstat, s.nk_cap);
    if (PROF && (rc = tm->end(g->stream))) return rc;
    return GC_OK;
}

}  // namespace

int run_event_maxmin(gc_graph *g, const RunParams &p, RunResult *r) {
    Scratch &s = g->s;
    const int64_t n = g->n;
    r->rounds = r->inner = r->launches = 0;
    if (n == 0) return GC_OK;
    int rc = fill_u32(s.C, GC_UNC, n, g->stream);  // Alg.5 L5
    if (rc) return rc;
    GC_CUDA_TRY(cudaMemsetAsync(s.S, 0, sizeof(uint32_t) * (size_t)n, g->stream));
    GC_CUDA_TRY(cudaMemsetAsync(s.ctr, 0, 48 * sizeof(unsigned long long), g->stream));
    const unsigned long long rem = (unsigned long long)n;
    GC_CUDA_TRY(cudaMemcpyAsync(s.ctr + kRem, &rem, sizeof(rem), cudaMemcpyHostToDevice, g->stream));
    r->launches += 1;
    const int grid = g->sm_count * 4;
    const int grid_dense =
        (int)std::max<int64_t>(1, std::min<int64_t>((n + kBlock - 1) / kBlock, (int64_t)g->sm_count * 8));
    const bool prof = p.prof && p.prof->on;
    EventTimer tm;
    int64_t k = 0;
    int64_t batch = p.batch_rounds > 0 ? p.batch_rounds : 8;
    for (;;) {
        rc = ensure_nk(g, k + batch + 1);
        if (rc) return rc;
        for (int64_t b = 0; b < batch; ++b, ++k) {
            rc = prof ? launch_round<true>(g, p, (uint32_t)k, grid, grid_dense, &tm)
                      : launch_round<false>(g, p, (uint32_t)k, grid, grid_dense, &tm);
            if (rc) return rc;
            r->launches += 4;
        }
        GC_CUDA_TRY(cudaGetLastError());
        GC_CUDA_TRY(cudaMemcpyAsync(s.host_pinned, s.nk + (k - batch), sizeof(int64_t) * batch,
                                    cudaMemcpyDeviceToHost, g->stream));
        GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
        if (prof && (rc = tm.drain(p.prof))) return rc;
        int64_t done_at = -1;
        for (int64_t b = 0; b < batch; ++b)
            if (s.host_pinned[b] == 0) {
                done_at = k - batch + b;
                break;
            }
        if (done_at >= 0) {
            r->rounds = done_at;
            break;
        }
        if (p.max_rounds > 0 && k >= p.max_rounds) {
            set_error("max-min colouring exceeded the round limit");
            return GC_ERR_TOO_LARGE;
        }
        if (p.batch_rounds <= 0) batch = std::min<int64_t>(batch * 2, 512);
    }
    r->inner = r->rounds;
    if (prof) {
        unsigned long long c[8];
        GC_CUDA_TRY(cudaMemcpy(c, s.ctr + kVisE, sizeof(c), cudaMemcpyDeviceToHost));
        const int64_t visE = (int64_t)c[0], visB = (int64_t)c[1], visN = (int64_t)c[2];
        const int64_t sumD = (int64_t)c[3];
        // algorithmic bytes: eval reads D (4 B), the
        // row offsets (16 B) and the witness state (16 B; not in the dense
        // round 0) per evaluated vertex, 4 B per scanned entry, and writes
        // either the witness state (16 B) or the colour + I entry (8 B);
        // notify reads I (4 B) and the row offsets (16 B) per coloured vertex
        // and 4 B per walked entry.
        const int64_t evalB = 4 * (sumD - n) + 16 * sumD + 16 * (sumD - n) + 4 * visE +
                              16 * (sumD - n) + 8 * n;
        p.prof->bytes[0] += evalB;
        p.prof->bytes[1] += 4 * visB;
        p.prof->bytes[2] += 20 * n + 4 * visN;  // notify + notify_big (walked entries)
        p.prof->visits += visE + visB;
    }
    return GC_OK;
}

}  // namespace gc
