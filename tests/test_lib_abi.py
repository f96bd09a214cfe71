"""libsp.so loads on a GPU-less host and exports every entry point include/sp.h declares;
host-only entry points (planner, geometry, footprints, status strings) work without a GPU."""
import ctypes
import os
import re

import pytest

import paper_conf_ppopp_baskaranbkrrs08_b200 as sp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _declared():
    txt = open(os.path.join(ROOT, "include", "sp.h")).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    return sorted(set(re.findall(r"\b(sp_[a-z0-9_]+)\s*\(", txt)))


def test_exports_every_declared_symbol():
    names = _declared()
    assert len(names) >= 17
    L = ctypes.CDLL(sp.LIB_PATH)
    for n in names:
        assert hasattr(L, n), n
    # and the binding wires every one of them
    assert set(names) <= set(sp.SYMBOLS), set(names) - set(sp.SYMBOLS)


def test_status_strings_and_version():
    assert sp.lib.sp_status_string(0) == b"SP_OK"
    assert sp.lib.sp_status_string(-3) == b"SP_ERR_CAPACITY"
    assert sp.lib.sp_status_string(-8) == b"SP_ERR_NCCL"
    assert sp.lib.sp_version() >= 100


def test_built_for_sm100a():
    import subprocess
    out = subprocess.run(["cuobjdump", "--list-elf", sp.LIB_PATH], capture_output=True, text=True).stdout
    assert "sm_100a" in out


def test_jacobi_plan_geometry_host_only():
    p = sp.jacobi1d_plan(1 << 26, 1024, 16, 0)
    assert p["passes"] == 64 and p["halo"] == 16
    assert p["space_tile"] % 4 == 0 and p["tiles"] == -(-(1 << 26) // p["space_tile"])
    assert sp.jacobi1d_plan(4096, 64, 16, 256)["space_tile"] == 256
    with pytest.raises(sp.SPError):
        sp.jacobi1d_plan(4096, 64, 0, 0)
    with pytest.raises(sp.SPError):
        sp.jacobi1d_plan(4096, 64, 16, 6)  # not a multiple of 4
    with pytest.raises(sp.SPError):
        sp.jacobi1d_plan(2, 64, 16, 0)


def test_jacobi_host_flags_len_host_only():
    """sp_jacobi1d_host's copy-engine route needs the persistent launch's tile flags, the unit
    counter and one ready flag per SP_JACOBI_HOST_CHUNK = 2^21 cells"""
    for n, tt in [(3, 64), (4099, 16), (1 << 26, 128), ((1 << 21) + 1, 48)]:
        p = sp.jacobi1d_plan(n, 1024, tt, 0)
        assert sp.jacobi1d_host_flags_len(n, 1024, tt) == p["persistent_tiles"] + 1 + -(-n // (1 << 21))
    with pytest.raises(sp.SPError):
        sp.jacobi1d_host_flags_len(2, 10, 16)


def test_jacobi_tile_footprint_closed_form():
    assert sp.jacobi1d_tile_footprint(100, 5, 0, 16) == (0, 20)
    assert sp.jacobi1d_tile_footprint(100, 5, 96, 16) == (91, 99)
    assert sp.jacobi1d_tile_footprint(100, 0, 32, 16) == (32, 47)


def test_me_ref_window():
    assert sp.me_ref_window(352, 288, 16, 0, 0) == ((0, 0), (31, 31))
    assert sp.me_ref_window(352, 288, 16, 5, 7) == ((112 - 16, 80 - 16), (112 + 31, 80 + 31))
    assert sp.me_ref_window(1920, 1080, 32, 119, 66) == ((1056 - 32, 1904 - 32), (1079, 1919))


def test_device_entry_points_reject_bad_args_without_gpu():
    # argument validation happens before any CUDA call
    assert sp.lib.sp_jacobi1d_timetiled(None, None, 10, 1, 16, 0, None, None) == -1
    assert sp.lib.sp_me_sad_search(None, None, 16, 16, 16, 0, 16, 1, 256, 8, 4, 0, 1, None, None, None, None) == -5
    assert sp.lib.sp_me_sad_search(None, None, 16, 16, 16, 0, 16, 1, 256, 16, 4, 0, 1, None, None, None, None) == -1


def test_struct_layouts_match_the_library():
    """The binding's ctypes structs have the C ABI's sizes (sp_abi_struct_sizes)."""
    order = [sp.sp_domain, sp.sp_ref, sp.sp_block, sp.sp_plan_opts, sp.sp_buffer, sp.sp_jacobi_plan,
             sp.sp_peer_links, sp.sp_tile_problem, sp.sp_tile_result, sp.sp_op, sp.sp_stmt_body, sp.sp_array_desc,
             sp.sp_exec_opts, sp.sp_exec_stats, sp.sp_me_gather_links]
    out = (ctypes.c_int64 * len(order))()
    assert sp.lib.sp_abi_struct_sizes(out, len(order)) == len(order)
    for cls, n in zip(order, out):
        assert ctypes.sizeof(cls) == n, (cls.__name__, ctypes.sizeof(cls), n)


def test_peer_entry_points_validate_before_cuda():
    """sp_jacobi1d_timetiled_peer(_fused): argument errors return SP_ERR_INVALID_ARG before any
    CUDA call (fake, never dereferenced, 16-byte-aligned pointers)."""
    L = sp.sp_peer_links()
    L.my_flags = 0x10000
    a, w, f = 0x20000, 0x40000, 0x60000
    fused = sp.lib.sp_jacobi1d_timetiled_peer_fused
    # no links / a == work / misaligned slab start / x range outside the domain
    assert fused(None, a, w, f, 100, 1000, 0, 1000, 10, 16, 0, None) == -1
    assert fused(ctypes.byref(L), a, a, f, 100, 1000, 0, 1000, 10, 16, 0, None) == -1
    assert fused(ctypes.byref(L), a, w, f, 100, 1000, 2, 900, 10, 16, 0, None) == -1
    assert fused(ctypes.byref(L), a, w, f, 100, 1000, 0, 1001, 10, 16, 0, None) == -1
    # a slab with a left neighbour but no mapped neighbour buffers
    assert fused(ctypes.byref(L), a, w, f, 100, 1000, 500, 500, 10, 16, 0, None) == -1
    # flags too short: tiles + 1 + 2 * passes entries are needed (one tile, 1 pass -> 4)
    assert fused(ctypes.byref(L), a, w, f, 3, 1000, 0, 1000, 10, 16, 0, None) == -1
    # zero steps is the identity (no launch)
    assert fused(ctypes.byref(L), a, w, f, 1, 1000, 0, 1000, 0, 16, 0, None) == 0
    per_pass = sp.lib.sp_jacobi1d_timetiled_peer
    assert per_pass(None, a, w, 1000, 0, 1000, 10, 16, 0, None) == -1
    assert per_pass(ctypes.byref(L), a, w, 1000, 500, 500, 10, 16, 0, None) == -1
