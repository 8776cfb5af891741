"""CPU-side checks of the C-ABI boundary (no compute calls need a GPU here).

* libppr.so loads and exports every function include/ppr.h declares;
* argument validation happens before any CUDA work, so the documented error
  codes can be checked on a machine without a GPU;
* the product library and the oracle share no code (no common symbols,
  neither imports the other).
"""
import ctypes
import os
import re
import subprocess

import numpy as np
import pytest

from paper_journals_pvldb_guolst17_b200 import build, ppr

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "ppr.h")


@pytest.fixture(scope="module")
def lib():
    build.build_lib()
    return ppr.load()


def _declared():
    src = open(HEADER).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(ppr_[a-z0-9_]+)\s*\(", src)))


def test_header_declares_the_documented_entry_points():
    names = _declared()
    assert {"ppr_create", "ppr_apply_batch", "ppr_query"} <= set(names)
    assert names == sorted(ppr.EXPORTS)


def test_library_exports_every_declared_symbol(lib):
    for name in _declared():
        assert hasattr(lib, name), name
    out = subprocess.run(["nm", "-D", "--defined-only", ppr.LIB_PATH], capture_output=True,
                         text=True, check=True).stdout
    exported = {l.split()[-1] for l in out.splitlines() if " T " in l}
    for name in _declared():
        assert name in exported, name


def test_status_strings(lib):
    for code, name in [(0, "PPR_OK"), (-1, "PPR_EINVAL"), (-2, "PPR_ERANGE"), (-3, "PPR_ENOENT"),
                       (-4, "PPR_ENOMEM"), (-5, "PPR_ECUDA"), (-6, "PPR_EPOISONED"),
                       (-7, "PPR_ENOCONV")]:
        assert lib.ppr_status_str(code).decode() == name


def _create(lib, n, src, dst, sources, alpha, eps):
    s = np.ascontiguousarray(src, dtype=np.uint32)
    d = np.ascontiguousarray(dst, dtype=np.uint32)
    so = np.ascontiguousarray(sources, dtype=np.uint32)
    u32p = ctypes.POINTER(ctypes.c_uint32)
    g = ppr.Graph(n=n, m=len(s), src=s.ctypes.data_as(u32p), dst=d.ctypes.data_as(u32p), undirected=0)
    h = ctypes.c_void_p()
    rc = lib.ppr_create(ctypes.byref(g), so.ctypes.data_as(u32p), len(so), alpha, eps, None,
                        ctypes.byref(h), None)
    return rc, h


@pytest.mark.parametrize("alpha,eps", [(0.0, 1e-6), (1.0, 1e-6), (-0.1, 1e-6), (0.15, 0.0),
                                       (0.15, -1.0), (0.15, float("inf")), (0.15, float("nan"))])
def test_create_rejects_bad_parameters_before_any_cuda_work(lib, alpha, eps):
    rc, h = _create(lib, 4, [0, 1], [1, 2], [0], alpha, eps)
    assert rc == ppr.PPR_EINVAL and not h.value


def test_create_rejects_bad_sources_and_ids(lib):
    assert _create(lib, 4, [0], [1], [0, 0], 0.15, 1e-6)[0] == ppr.PPR_EINVAL   # duplicate
    assert _create(lib, 4, [0], [1], [4], 0.15, 1e-6)[0] == ppr.PPR_ERANGE      # source >= n
    assert _create(lib, 4, [0], [7], [0], 0.15, 1e-6)[0] == ppr.PPR_ERANGE      # arc id >= n
    assert _create(lib, 0, [], [], [0], 0.15, 1e-6)[0] == ppr.PPR_EINVAL        # n = 0
    assert _create(lib, 4, [0], [1], [], 0.15, 1e-6)[0] == ppr.PPR_EINVAL       # no sources


def test_null_handle_calls_are_einval(lib):
    assert lib.ppr_apply_batch(None, None, None, 0, None, None, 0, 0, None) == ppr.PPR_EINVAL
    assert lib.ppr_destroy(None) == ppr.PPR_EINVAL
    assert lib.ppr_set_option(None, 1, 0) == ppr.PPR_EINVAL


def test_product_and_oracle_share_no_code():
    import oracle
    oracle.build()
    def syms(path):
        out = subprocess.run(["nm", "-D", "--defined-only", path], capture_output=True, text=True,
                             check=True).stdout
        return {l.split()[-1] for l in out.splitlines() if " T " in l}
    a = syms(ppr.LIB_PATH)
    b = syms(os.path.join(ROOT, "oracle", "liboracle.so"))
    assert not (a & b), a & b
    pkg = os.path.join(ROOT, "paper_journals_pvldb_guolst17_b200")
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".c", ".h")):
                text = open(os.path.join(dirpath, f), errors="ignore").read()
                assert not re.search(r"^\s*(import|from)\s+oracle\b", text, re.M), f
                assert "ppr_oracle" not in text, f
    for f in os.listdir(os.path.join(ROOT, "oracle")):
        if f.endswith((".py", ".c", ".h")):
            text = open(os.path.join(ROOT, "oracle", f), errors="ignore").read()
            assert not re.search(r"^\s*(import|from)\s+paper_journals_pvldb_guolst17_b200", text,
                                 re.M), f
            assert not re.search(r'#\s*include\s*[<"][^>"]*ppr\.h', text), f
            assert not re.search(r'#\s*include\s*[<"][^>"]*csrc', text), f
