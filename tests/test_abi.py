"""The C-ABI library builds, loads and exports every symbol include/gc.h
declares; without a GPU every compute entry point fails loudly (no CPU
fallback).  Runs on the CPU-only dev box (no compute calls)."""
import ctypes
import os
import re
import subprocess

import pytest

import paper_conf_ipps_osamatybo19_b200 as gcb
from paper_conf_ipps_osamatybo19_b200 import build as gbuild

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "gc.h")


def declared_functions():
    text = open(HEADER).read()
    text = re.sub(r"/\*.*?\*/", "", text, flags=re.S)
    return sorted(set(re.findall(r"\b(gc_[a-z_0-9]+)\s*\(", text)) - {"gc_graph"})


@pytest.fixture(scope="module")
def libgc():
    gbuild.build()
    return gcb.lib()


def test_header_declares_the_boundary():
    names = declared_functions()
    for must in ("gc_create_csr", "gc_color", "gc_destroy", "gc_color_ex", "gc_last_error",
                 "gc_set_stream", "gc_create_csr_dist", "gc_priorities", "gc_count_colors"):
        assert must in names
    assert set(names) == set(gcb.EXPORTS)


def test_library_exports_every_declared_symbol(libgc):
    out = subprocess.run(["nm", "-D", "--defined-only", gbuild.OUT], capture_output=True,
                         text=True, check=True).stdout
    exported = set(re.findall(r" T (gc_\w+)", out))
    missing = set(declared_functions()) - exported
    assert not missing, missing
    for name in declared_functions():
        assert hasattr(libgc, name)


def test_library_is_sm100a_only(libgc):
    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "--list-elf", gbuild.OUT],
                         capture_output=True, text=True).stdout
    assert "sm_100a" in out


def _compile_and_run(src: str) -> str:
    import tempfile
    with tempfile.TemporaryDirectory() as d:
        c, exe = os.path.join(d, "t.c"), os.path.join(d, "t")
        open(c, "w").write(src)
        subprocess.check_call(["gcc", "-I" + os.path.join(ROOT, "include"), "-o", exe, c])
        return subprocess.check_output([exe]).decode()


def test_struct_layouts_match_header():
    """sizeof / offsetof of every field of gc_options and gc_stats as the C
    compiler lays out include/gc.h, against the binding's ctypes structures."""
    lines = ['#include <stdio.h>', '#include <stddef.h>', '#include "gc.h"', 'int main(void){']
    for st in (gcb.gc_options, gcb.gc_stats):
        name = st.__name__
        lines.append(f'printf("{name} size %zu\\n", sizeof({name}));')
        for f, _ in st._fields_:
            lines.append(f'printf("{name} {f} %zu\\n", offsetof({name}, {f}));')
    lines.append("return 0;}")
    got = {}
    for ln in _compile_and_run("\n".join(lines) + "\n").splitlines():
        st, f, v = ln.split()
        got[(st, f)] = int(v)
    for st in (gcb.gc_options, gcb.gc_stats):
        assert got[(st.__name__, "size")] == ctypes.sizeof(st), st.__name__
        for f, _ in st._fields_:
            assert got[(st.__name__, f)] == getattr(st, f).offset, (st.__name__, f)


def test_fails_loudly_without_gpu(libgc):
    import torch
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    assert libgc.gc_last_error() in (b"",) or isinstance(libgc.gc_last_error(), bytes)
    ro = torch.tensor([0, 1, 2], dtype=torch.int64)
    ci = torch.tensor([1, 0], dtype=torch.int32)
    with pytest.raises(gcb.GCError) as e:
        gcb.Graph(2, ro, ci)
    assert e.value.code == -5 and "CUDA" in str(e.value) or "device" in str(e.value)
    with pytest.raises(gcb.GCError):
        gcb.priorities(1, 0, 0, 4, torch.empty(4, dtype=torch.int32))


def test_argument_errors_need_no_device(libgc):
    h = ctypes.c_void_p()
    assert libgc.gc_create_csr(2, 2, None, None, 0, ctypes.byref(h)) == -1
    assert libgc.gc_create_csr(-1, 0, None, None, 0, ctypes.byref(h)) == -1
    assert libgc.gc_create_csr(2, 0, None, None, 0, None) == -1
    assert b"NULL" in libgc.gc_last_error() or b"bad" in libgc.gc_last_error()
    libgc.gc_destroy(None)  # NULL-safe
    assert libgc.gc_color(None, 1, 0, None) == -1
    assert libgc.gc_set_stream(None, None) == -1


def test_variant_codes_match_header():
    # the binding's variant codes are the header's macros, evaluated by the C compiler
    src = ('#include <stdio.h>\n#include "gc.h"\nint main(void){printf("%d %d %d %d %d %d %d %d\\n",'
           'GC_MAXMIN, GC_LUBY_MIS, GC_MULTIHASH(4), GC_IS_ALG2, GC_JP_ALG4, GC_HASH_IS(8),'
           'GC_HASH_TABLE_MAX, GC_LDF(GC_JP_ALG4));return 0;}\n')
    import tempfile
    with tempfile.TemporaryDirectory() as d:
        c, exe = os.path.join(d, "v.c"), os.path.join(d, "v")
        open(c, "w").write(src)
        subprocess.check_call(["gcc", "-I" + os.path.join(ROOT, "include"), "-o", exe, c])
        got = [int(x) for x in subprocess.check_output([exe]).split()]
    assert got == [gcb.MAXMIN, gcb.LUBY_MIS, gcb.MULTIHASH(4), gcb.IS_ALG2, gcb.JP_ALG4,
                   gcb.HASH_IS(8), gcb.HASH_TABLE_MAX, gcb.LDF(gcb.JP_ALG4)]


def test_binding_rejects_short_buffers():
    """The binding checks every buffer the C side reads or writes against the
    sizes it passes: a short array raises ValueError before any
    call reaches libgc -- no out-of-bounds device or host access."""
    import numpy as np
    import torch
    ro = torch.tensor([0, 1, 2], dtype=torch.int64)
    ci = torch.tensor([1, 0], dtype=torch.int32)
    with pytest.raises(ValueError, match="row_offsets"):
        gcb.Graph(3, ro, ci)  # n + 1 = 4 offsets needed
    with pytest.raises(ValueError, match="row_offsets"):
        gcb.loopback_graph(1, ro, ci, 2)
    with pytest.raises(ValueError, match="out"):
        gcb.priorities(1, 0, 0, 8, torch.empty(4, dtype=torch.int32))
    with pytest.raises(ValueError, match="out"):
        gcb.priorities(1, 0, 0, 8, np.empty(7, dtype=np.uint32))
    g = gcb.Graph._from_handle(ctypes.c_void_p(), 10, 0)  # no device needed: rejected first
    with pytest.raises(ValueError, match="out"):
        g.color(1, gcb.MAXMIN, torch.empty(9, dtype=torch.int32))
    g.local_len = 4  # a rank's owned range (dist_graph)
    with pytest.raises(ValueError, match="out"):
        g.color(1, gcb.MAXMIN, torch.empty(3, dtype=torch.int32), flags=gcb.OUT_LOCAL_SLICE)
    g._h = ctypes.c_void_p()
