// gc_alloc.cu -- the library's device / pinned-host memory cache.
//
// A colouring handle needs ~3 GB of device memory at R-MAT scale 24 (the CSR
// copy, colours, the event-mode witness state and queues).  cudaMalloc of
// that much maps pages (milliseconds) and cudaFree synchronises the device,
// so a user that creates, colours and destroys a handle per graph (the e2e
// path of bench.py) would pay both every time.  Freed blocks are kept in a
// per-device free list keyed by size and handed out again (best fit within
// 1/8 slack); a failing cudaMalloc first returns every cached block of that
// device to the driver and retries.  gc_trim() releases the cache.
//
// Contract: a block is released (dfree) only when no device work that uses it
// is still pending -- gc_destroy synchronises the handle's stream first.
// GC_NO_CACHE=1 in the environment disables caching (plain cudaMalloc/Free).
#include <cstdlib>
#include <map>
#include <mutex>
#include <unordered_map>

#include "gc_internal.cuh"

namespace gc {

namespace {

constexpr int kMaxDev = 64;

struct Block {
    size_t bytes;
    int dev;  // -1: pinned host
};

struct Cache {
    std::mutex m;
    std::multimap<size_t, void *> free_dev[kMaxDev];
    std::multimap<size_t, void *> free_host;
    std::unordered_map<void *, Block> live;
    size_t cached_dev[kMaxDev] = {};
    size_t cached_host = 0;
    int enabled = -1;
};

Cache &cache() {
    static Cache *c = new Cache();  // never destroyed: blocks may be freed at exit
    return *c;
}

bool caching(Cache &c) {
    if (c.enabled < 0) {
        const char *e = std::getenv("GC_NO_CACHE");
        c.enabled = (e && e[0] && e[0] != '0') ? 0 : 1;
    }
    return c.enabled == 1;
}

size_t round_size(size_t b) {
    if (b == 0) b = 1;
    if (b < ((size_t)1 << 20)) return (b + 511) & ~(size_t)511;
    return (b + ((size_t)2 << 20) - 1) & ~(((size_t)2 << 20) - 1);
}

// take a cached block of at least `sz` bytes and at most sz + sz/8 (locked)
void *take(std::multimap<size_t, void *> &fl, size_t sz, size_t *got) {
    auto it = fl.lower_bound(sz);
    if (it == fl.end() || it->first > sz + sz / 8) return nullptr;
    void *p = it->second;
    *got = it->first;
    fl.erase(it);
    return p;
}

void release_dev_locked(Cache &c, int dev) {
    if (dev < 0 || dev >= kMaxDev) return;
    for (auto &kv : c.free_dev[dev]) cudaFree(kv.second);
    c.free_dev[dev].clear();
    c.cached_dev[dev] = 0;
}

}  // namespace

cudaError_t dmalloc_raw(void **p, size_t bytes) {
    Cache &c = cache();
    int dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return e;
    const size_t sz = round_size(bytes);
    std::lock_guard<std::mutex> lk(c.m);
    if (caching(c) && dev < kMaxDev) {
        size_t got = 0;
        if (void *q = take(c.free_dev[dev], sz, &got)) {
            c.cached_dev[dev] -= got;
            c.live[q] = Block{got, dev};
            *p = q;
            return cudaSuccess;
        }
    }
    e = cudaMalloc(p, sz);
    if (e == cudaErrorMemoryAllocation) {
        cudaGetLastError();  // clear the sticky-free error state
        release_dev_locked(c, dev);
        e = cudaMalloc(p, sz);
    }
    if (e != cudaSuccess) {
        *p = nullptr;
        return e;
    }
    c.live[*p] = Block{sz, dev};
    return cudaSuccess;
}

void dfree(void *p) {
    if (!p) return;
    Cache &c = cache();
    std::lock_guard<std::mutex> lk(c.m);
    auto it = c.live.find(p);
    if (it == c.live.end()) {  // not ours (should not happen): hand it to the driver
        cudaFree(p);
        return;
    }
    const Block b = it->second;
    c.live.erase(it);
    if (!caching(c) || b.dev < 0 || b.dev >= kMaxDev) {
        cudaFree(p);
        return;
    }
    c.free_dev[b.dev].emplace(b.bytes, p);
    c.cached_dev[b.dev] += b.bytes;
}

cudaError_t hmalloc_raw(void **p, size_t bytes) {
    Cache &c = cache();
    const size_t sz = round_size(bytes);
    std::lock_guard<std::mutex> lk(c.m);
    if (caching(c)) {
        size_t got = 0;
        if (void *q = take(c.free_host, sz, &got)) {
            c.cached_host -= got;
            c.live[q] = Block{got, -1};
            *p = q;
            return cudaSuccess;
        }
    }
    cudaError_t e = cudaMallocHost(p, sz);
    if (e != cudaSuccess) {
        *p = nullptr;
        return e;
    }
    c.live[*p] = Block{sz, -1};
    return cudaSuccess;
}

void hfree(void *p) {
    if (!p) return;
    Cache &c = cache();
    std::lock_guard<std::mutex> lk(c.m);
    auto it = c.live.find(p);
    if (it == c.live.end()) {
        cudaFreeHost(p);
        return;
    }
    const Block b = it->second;
    c.live.erase(it);
    if (!caching(c)) {
        cudaFreeHost(p);
        return;
    }
    c.free_host.emplace(b.bytes, p);
    c.cached_host += b.bytes;
}

size_t cached_bytes() {
    Cache &c = cache();
    std::lock_guard<std::mutex> lk(c.m);
    size_t s = c.cached_host;
    for (int d = 0; d < kMaxDev; ++d) s += c.cached_dev[d];
    return s;
}

}  // namespace gc

extern "C" int gc_trim(void) {
    gc::Cache &c = gc::cache();
    std::lock_guard<std::mutex> lk(c.m);
    int cur = 0;
    cudaGetDevice(&cur);
    for (int d = 0; d < gc::kMaxDev; ++d) {
        if (c.free_dev[d].empty()) continue;
        cudaSetDevice(d);
        gc::release_dev_locked(c, d);
    }
    cudaSetDevice(cur);
    for (auto &kv : c.free_host) cudaFreeHost(kv.second);
    c.free_host.clear();
    c.cached_host = 0;
    return GC_OK;
}
