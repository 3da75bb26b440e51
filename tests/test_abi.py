"""CPU-only checks of the C-ABI library: it builds for sm_100a, loads, and exports
every entry point include/ar.h declares (no compute calls without a GPU)."""
import ctypes
import os
import re
import subprocess

import numpy as np

from tests._layout import unpack_packed, unpack_sliced

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "ar.h")


def declared_functions():
    text = open(HEADER).read()
    text = re.sub(r"/\*.*?\*/", "", text, flags=re.S)
    names = re.findall(r"^\s*(?:const\s+)?[A-Za-z_][A-Za-z0-9_]*\s*\**\s*(ar_[a-z0-9_]+)\s*\(", text, flags=re.M)
    return sorted(set(names))


def test_header_declares_boundary():
    names = declared_functions()
    for must in ["ar_decompose_plan", "ar_decompose", "ar_approx_select", "ar_refine", "ar_sum",
                 "ar_refine_sum", "ar_select_refine_sum", "ar_dist_init", "ar_dist_offsets", "ar_dist_sum"]:
        assert must in names


def test_library_exports_every_declared_symbol():
    from paper_conf_icde_pirkmk14_b200 import _ar
    lib = _ar.load()
    path = _ar.lib_path()
    out = subprocess.run(["nm", "-D", "--defined-only", path], capture_output=True, text=True, check=True).stdout
    exported = set(re.findall(r"\sT\s(ar_[a-z0-9_]+)$", out, flags=re.M))
    missing = [n for n in declared_functions() if n not in exported]
    assert not missing, missing
    for n in declared_functions():
        assert hasattr(lib, n)
    # every declared symbol has a binding with the same name
    assert set(declared_functions()) <= set(_ar.SIGNATURES)


def test_library_is_sm100a():
    from paper_conf_icde_pirkmk14_b200 import _ar
    out = subprocess.run(["cuobjdump", "--list-elf", _ar.lib_path()], capture_output=True, text=True).stdout
    assert "sm_100a" in out
    sass = subprocess.run(["cuobjdump", "-sass", _ar.lib_path()], capture_output=True, text=True).stdout
    assert "UBLKCP" in sass            # TMA bulk copies in the scan kernels


def test_host_only_entry_points():
    from paper_conf_icde_pirkmk14_b200 import _ar
    lib = _ar.load()
    assert lib.ar_status_str(0) == b"AR_OK" and lib.ar_status_str(2) == b"AR_ERR_RANGE"
    assert b"sm_100a" in lib.ar_version()
    # per-tile counts + offsets and the tile-local candidate slices (8 B per row)
    assert _ar.ar_select_ws_bytes(4096) >= 8 * 4096 and _ar.ar_select_ws_bytes(4097) >= 8 * 4097
    assert _ar.ar_refine_ws_bytes(2048) == 16 + 8
    assert _ar.ar_dist_unique_id_bytes() == 128
    assert _ar.ar_minmax_ws_bytes(100) == 64 + 4 * 100   # header + one Y major per candidate
    assert ctypes.sizeof(_ar.ColumnDesc) == 64


def test_host_validation_without_gpu():
    from paper_conf_icde_pirkmk14_b200 import _ar
    import pytest
    with pytest.raises(_ar.ARError) as e:
        _ar.ar_decompose_plan(None, 10, 24, 0, 0, 0, 0, None, 0, None)
    assert e.value.status == _ar.AR_ERR_INVALID
    with pytest.raises(_ar.ARError) as e:
        _ar.ar_decompose_plan(None, 0, 33, 0, 0, 0, 0, None, 0, None)
    assert e.value.status == _ar.AR_ERR_INVALID
    with pytest.raises(_ar.ARError) as e:
        _ar.ar_approx_select([], 0, _ar.Cands(), None, 0, None)
    assert e.value.status == _ar.AR_ERR_INVALID
    # the PDL flags need a workspace; a short workspace is a range error (checked before any CUDA call)
    with pytest.raises(_ar.ARError) as e:
        _ar.ar_select_refine_sum_ws([], [], _ar.AR_SRS_PDL, None, None, 0, None)
    assert e.value.status == _ar.AR_ERR_INVALID
    with pytest.raises(_ar.ARError) as e:
        _ar.ar_select_refine_sum_ws([], [], 0, None, 16, 8, None)
    assert e.value.status == _ar.AR_ERR_RANGE
    assert _ar.ar_select_refine_sum_ws_bytes() >= 128 + 296 * 32


def test_layout_decoders_by_hand():
    # PACKED w=3, values 1,2,3,4,5 -> bits 001 010 011 100 101 LSB-first = 0b101_100_011_010_001
    word = 0b101100011010001
    buf = np.array([word, 0], dtype="<u4").tobytes()
    assert unpack_packed(buf, 5, 3).tolist() == [1, 2, 3, 4, 5]
    # SLICED w=2: rows 0..31, value of row l = l % 4 -> plane0 = 0xAAAAAAAA, plane1 = 0xCCCCCCCC
    buf = np.array([0xAAAAAAAA, 0xCCCCCCCC], dtype="<u4").tobytes()
    assert unpack_sliced(buf, 32, 2).tolist() == [l % 4 for l in range(32)]
