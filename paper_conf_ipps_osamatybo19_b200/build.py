"""Build libgc.so in-tree with nvcc for sm_100a (no JIT cache: the .so travels
with the repo snapshot to the GPU box).  Usage: python -m paper_conf_ipps_osamatybo19_b200.build"""
from __future__ import annotations

import glob
import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(HERE)
CSRC = os.path.join(HERE, "csrc")
OUT = os.path.join(HERE, "libgc.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")


def nccl_dirs():
    try:
        import nvidia.nccl as m  # torch's bundled NCCL (2.28.x)
        base = list(m.__path__)[0]
        inc, libd = os.path.join(base, "include"), os.path.join(base, "lib")
        if os.path.exists(os.path.join(inc, "nccl.h")):
            return inc, libd
    except Exception:
        pass
    return None, None


def sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")))


def needs_build() -> bool:
    if not os.path.exists(OUT):
        return True
    t = os.path.getmtime(OUT)
    deps = sources() + glob.glob(os.path.join(CSRC, "*.cuh")) + [os.path.join(ROOT, "include", "gc.h")]
    return any(os.path.getmtime(p) > t for p in deps)


OBJ = os.path.join(ROOT, "build", "obj")


def build(force: bool = False, verbose: bool = False, out: str = OUT, defines=()) -> str:
    """One object per .cu (compiled in parallel, rebuilt when the source or a
    header is newer), then one nvcc link step into `out`."""
    if not force and out == OUT and not defines and not needs_build():
        return out
    from concurrent.futures import ThreadPoolExecutor

    inc, libd = nccl_dirs()
    flags = [NVCC, "-gencode", "arch=compute_100a,code=sm_100a", "-O3", "-lineinfo", "-std=c++17",
             "-Xcompiler", "-fPIC", "-I" + os.path.join(ROOT, "include")]
    flags += ["-D" + d for d in defines]
    if inc:
        flags += ["-DGC_HAVE_NCCL=1", "-I" + inc]
    if verbose:
        flags += ["-Xptxas", "-v"]
    tag = "_".join(d.replace("=", "") for d in defines) or "default"
    odir = os.path.join(OBJ, tag)
    os.makedirs(odir, exist_ok=True)
    hdrs = glob.glob(os.path.join(CSRC, "*.cuh")) + [os.path.join(ROOT, "include", "gc.h")]
    t_hdr = max(os.path.getmtime(h) for h in hdrs)

    def one(src):
        obj = os.path.join(odir, os.path.basename(src) + ".o")
        if force or not os.path.exists(obj) or os.path.getmtime(obj) < max(os.path.getmtime(src), t_hdr):
            tmpo = obj + f".tmp{os.getpid()}"
            subprocess.check_call(flags + ["-c", "-o", tmpo, src])
            os.replace(tmpo, obj)
        return obj

    with ThreadPoolExecutor(max_workers=min(8, os.cpu_count() or 1)) as ex:
        objs = list(ex.map(one, sources()))
    link = [NVCC, "-gencode", "arch=compute_100a,code=sm_100a", "-shared", "-Xcompiler", "-fPIC",
            "-Xlinker", "--no-undefined"]
    if inc:
        link += ["-L" + libd, "-Xlinker", "-rpath=" + libd, "-l:libnccl.so.2"]
    tmp = out + f".tmp{os.getpid()}"
    subprocess.check_call(link + ["-o", tmp] + objs)
    os.replace(tmp, out)
    return out


if __name__ == "__main__":
    # python -m paper_conf_ipps_osamatybo19_b200.build [--force] [-v] [-DNAME=V ... --out PATH]
    defs = [a[2:] for a in sys.argv[1:] if a.startswith("-D")]
    o = sys.argv[sys.argv.index("--out") + 1] if "--out" in sys.argv else OUT
    print(build(force="--force" in sys.argv, verbose="-v" in sys.argv, out=o, defines=defs))
