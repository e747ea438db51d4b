"""CPU-side checks of the C ABI: the library builds, loads and exports every declared symbol."""
import ctypes as C
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "gpma.h")


def _declared():
    txt = open(HEADER).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    return sorted(set(re.findall(r"\b(gpma_[a-z0-9_]+)\s*\(", txt)))


@pytest.fixture(scope="module")
def lib():
    from paper_journals_pvldb_shalht17_b200.buildlib import build
    build()
    from paper_journals_pvldb_shalht17_b200 import lib as load
    return load()


def test_header_declares_the_north_star_entry_points():
    names = _declared()
    for n in ["gpma_create", "gpma_update_batch", "gpma_bfs", "gpma_cc", "gpma_pagerank", "gpma_export_csr"]:
        assert n in names


def test_every_declared_symbol_is_exported(lib):
    from paper_journals_pvldb_shalht17_b200.buildlib import LIB
    out = subprocess.check_output(["nm", "-D", "--defined-only", LIB]).decode()
    exported = set(re.findall(r"\bT (gpma_\w+)", out))
    missing = [n for n in _declared() if n not in exported]
    assert not missing, f"declared but not exported: {missing}"
    for n in _declared():
        assert hasattr(lib, n)


def test_library_is_sm100a(lib):
    from paper_journals_pvldb_shalht17_b200.buildlib import LIB
    out = subprocess.check_output(["/usr/local/cuda/bin/cuobjdump", "--list-elf", LIB]).decode()
    assert "sm_100a" in out


def test_host_only_entry_points(lib):
    from paper_journals_pvldb_shalht17_b200.gpma import gpma_config
    cfg = gpma_config()
    lib.gpma_config_default(C.byref(cfg))
    assert (cfg.rho_leaf_bp, cfg.rho_root_bp, cfg.tau_leaf_bp, cfg.tau_root_bp) == (800, 4000, 9200, 8000)
    assert cfg.init_density_bp == 6000 and cfg.struct_size == C.sizeof(gpma_config)
    assert lib.gpma_status_string(3) == b"reserved key or value"
    assert lib.gpma_last_error(None) == b"null handle"
    assert lib.gpma_destroy(None) == 1


def test_null_arguments_rejected_without_gpu(lib):
    h = C.c_void_p()
    assert lib.gpma_create(0, None, None, 0, None, None, C.byref(h)) == 1
    assert lib.gpma_update_batch(None, None, None, 0, 0, None) == 1


def test_no_cpu_fallback_when_no_device(lib):
    """Without a CUDA device the product path fails loudly (no CPU fallback)."""
    import torch
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    h = C.c_void_p()
    st = lib.gpma_create(4, None, None, 0, None, None, C.byref(h))
    assert st != 0 and not h.value


def test_product_does_not_import_oracle():
    pkg = os.path.join(ROOT, "paper_journals_pvldb_shalht17_b200")
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                txt = open(os.path.join(dirpath, f)).read()
                assert "oracle" not in re.sub(r"(#|//).*", "", txt).lower().replace("oracle/", ""), f
