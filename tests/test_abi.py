"""The C-ABI library loads and exports every symbol include/hj.h declares (CPU, no compute)."""
import ctypes
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "hj.h")


def declared_symbols():
    src = open(HEADER).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(hj_[a-z_]+)\s*\(", src)))


def test_header_symbols_nonempty():
    syms = declared_symbols()
    assert {"hj_create", "hj_join", "hj_destroy", "hj_join_host", "hj_partition"} <= set(syms)


def test_library_exports_every_declared_symbol():
    import paper_conf_icde_sioulasckaa19_b200 as hj

    lib = ctypes.CDLL(hj.LIB_PATH)
    for s in declared_symbols():
        assert hasattr(lib, s), f"libhj.so does not export {s}"
    assert set(declared_symbols()) == set(hj.EXPORTS)


def test_library_is_sm100a():
    import paper_conf_icde_sioulasckaa19_b200 as hj

    out = subprocess.run(["cuobjdump", "--list-elf", hj.LIB_PATH], capture_output=True, text=True).stdout
    assert "sm_100a" in out
    assert "sm_100a" in hj.version()


def test_create_without_gpu_fails_loudly():
    import torch

    import paper_conf_icde_sioulasckaa19_b200 as hj

    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    with pytest.raises(hj.HJError) as ei:
        hj.Context(0, 4, 4)
    assert ei.value.code in (-4, -1)


def test_unsupported_widths_rejected():
    import paper_conf_icde_sioulasckaa19_b200 as hj

    h = ctypes.c_void_p()
    assert hj.lib().hj_create(ctypes.byref(h), 0, 4, 8, None) == -2
    assert b"4/8" in hj.lib().hj_last_error(None)


def test_product_package_never_imports_oracle():
    pkg = os.path.join(ROOT, "paper_conf_icde_sioulasckaa19_b200")
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                txt = open(os.path.join(dirpath, f)).read()
                assert "oracle" not in re.sub(r"(#|//).*", "", txt).lower().replace("oracle/", ""), f
