"""Python binding of libsp (include/sp.h) — argument marshalling only.

B200-native (sm_100a) implementation of the data-parallel hot path of Baskaran et al.,
"Automatic Data Movement and Computation Mapping for Multi-level Parallel Architectures
with Explicitly Managed Memories", PPoPP'08: staged multi-level-tiled execution of the
paper's two GPU workloads (time-tiled 1-D Jacobi, MPEG-4 full-search SAD motion
estimation) plus the paper's buffer planner (Alg. 1 / Alg. 2 / §3.1.2-3.1.3).

Every step of the path runs in libsp.so (CUDA kernels + C++ host code); this module only
converts arguments.  PyTorch supplies device memory, streams and process groups.  There is
no CPU fallback: importing this package without the built library raises ImportError, and
the device entry points raise SPError when no usable device is present.

C entry point -> Python name (same names, `sp_` prefix dropped):
  sp_plan_buffers             -> plan_buffers(block, ...)
  sp_jacobi1d_plan            -> jacobi1d_plan(n, steps, time_tile, space_tile)
  sp_jacobi1d_tile_footprint  -> jacobi1d_tile_footprint(n, h, x0, space_tile)
  sp_jacobi1d_timetiled       -> jacobi1d_timetiled(a, steps, ...)     (device tensor, in place)
  sp_jacobi1d_timetiled_fused -> jacobi1d_timetiled_fused(a, steps, ...) (one persistent launch)
  sp_jacobi1d_timetiled_stream -> jacobi1d_timetiled_stream(inp, out, steps, ...) (device or pinned host)
  sp_jacobi1d_host            -> Jacobi1DHost(n, steps, ...).run(a_pinned)  (the e2e public call)
  sp_jacobi1d_resident        -> jacobi1d_resident(a, steps)   (small domains: one cluster)
  sp_jacobi1d_pass_segment    -> jacobi1d_pass_segment(...)
  sp_jacobi1d_timetiled_loopback -> jacobi1d_timetiled_loopback(...)
  sp_jacobi1d_timetiled_dist  -> Comm.jacobi1d_timetiled_dist(...)
  sp_me_sad_search            -> me_sad_search(ref, cur, ...)          (device tensors)
  sp_me_ref_window            -> me_ref_window(...)
  sp_me_search_host           -> MESearchHost(F, W, H, pitch, R).run(frames_pinned)  (the e2e public call)
  sp_me_sad_search_range      -> me_sad_search_range(frames, ...)      (one rank's range of a batch)
  sp_me_sad_search_gather     -> MEShard(...).run()                    (sharded batch, fused peer all-gather)
  sp_me_sad_search_dist       -> Comm.me_sad_search_dist(...)          (same, NCCL broadcast baseline)
  sp_get_unique_id / sp_comm_init / sp_comm_destroy / sp_allgather -> Comm
Host-buffer convenience (the end-to-end public API used for bench.py's `e2e`):
  jacobi1d(host_array, steps, ...), me_search(host_frames, ...)
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

__all__ = [
    "SPError", "lib", "plan_buffers", "jacobi1d_plan", "jacobi1d_tile_footprint", "jacobi1d_timetiled",
    "jacobi1d_pass_segment", "jacobi1d_timetiled_loopback", "me_sad_search", "me_ref_window", "me_search_sequence",
    "jacobi1d", "me_search", "Comm", "jacobi1d_timetiled_fused", "jacobi1d_timetiled_stream", "Jacobi1DHost", "MESearchHost", "jacobi1d_resident", "get_unique_id", "MEShard", "Prepared", "me_search_prepared", "jacobi1d_resident_prepared", "me_sad_search_range", "PER_ARRAY", "COMPONENTS", "halo_of",
]

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("SP_LIB") or os.path.join(_HERE, "libsp.so")

PER_ARRAY = 0
COMPONENTS = 1
MAX_RANK = 8

i32, i64, f64 = ctypes.c_int32, ctypes.c_int64, ctypes.c_double
vp = ctypes.c_void_p


class sp_domain(ctypes.Structure):
    _fields_ = [("depth", i32), ("n_rows", i32), ("rows", ctypes.POINTER(i64))]


class sp_ref(ctypes.Structure):
    _fields_ = [("stmt", i32), ("array", i32), ("is_write", i32), ("rank", i32), ("rows", ctypes.POINTER(i64))]


class sp_block(ctypes.Structure):
    _fields_ = [("n_params", i32), ("n_stmts", i32), ("n_refs", i32), ("reserved", i32),
                ("params", ctypes.POINTER(i64)), ("stmts", ctypes.POINTER(sp_domain)), ("refs", ctypes.POINTER(sp_ref))]


class sp_plan_opts(ctypes.Structure):
    _fields_ = [("mode", i32), ("reuse_filter", i32), ("delta", f64), ("mup_elems", i64), ("max_points", i64),
                ("compress", i32), ("reserved", i32)]


class sp_buffer(ctypes.Structure):
    _fields_ = [("array", i32), ("rank", i32), ("beneficial", i32), ("n_refs", i32),
                ("lb", i64 * MAX_RANK), ("ub", i64 * MAX_RANK), ("size", i64), ("v_in_ub", i64), ("v_out_ub", i64),
                ("in_lb", i64 * MAX_RANK), ("in_ub", i64 * MAX_RANK), ("in_count", i64),
                ("out_lb", i64 * MAX_RANK), ("out_ub", i64 * MAX_RANK), ("out_count", i64),
                ("in_dense", i32), ("out_dense", i32), ("overlap", i64), ("union_count", i64),
                ("n_dims", i32), ("kept_mask", i32)]


class sp_jacobi_plan(ctypes.Structure):
    _fields_ = [("n", i64), ("steps", i32), ("time_tile", i32), ("halo", i32), ("passes", i32), ("space_tile", i64),
                ("tiles", i64), ("grid", i32), ("threads", i32), ("smem_bytes", i32), ("cells_per_thread", i32),
                ("persistent_space_tile", i64), ("persistent_tiles", i64)]


class sp_peer_links(ctypes.Structure):
    _fields_ = [("left_bufs", vp * 2), ("right_bufs", vp * 2), ("left_n_local", i64), ("right_n_local", i64),
                ("left_flags", vp), ("right_flags", vp), ("my_flags", vp), ("epoch0", ctypes.c_uint64)]


ME_MAX_RANKS = 8


class sp_me_gather_links(ctypes.Structure):
    _fields_ = [("nranks", i32), ("rank", i32), ("mv", vp * ME_MAX_RANKS), ("sad", vp * ME_MAX_RANKS),
                ("flags", vp * ME_MAX_RANKS), ("epoch", ctypes.c_uint64)]


class sp_op(ctypes.Structure):
    _fields_ = [("op", i32), ("ref", i32), ("value", ctypes.c_float), ("reserved", i32)]


class sp_stmt_body(ctypes.Structure):
    _fields_ = [("write_ref", i32), ("n_ops", i32), ("ops", ctypes.POINTER(sp_op)), ("beta", ctypes.POINTER(i32))]


class sp_array_desc(ctypes.Structure):
    _fields_ = [("data", vp), ("rank", i32), ("reserved", i32), ("extent", i64 * 8)]


class sp_exec_opts(ctypes.Structure):
    _fields_ = [("n_tiles", i32), ("tiles_per_cta", i32), ("tile_params", ctypes.POINTER(i64)), ("hoist", i32),
                ("reuse_filter", i32), ("max_points", i64), ("movement", i32), ("dry_run", i32),
                ("live_out", ctypes.POINTER(i32)), ("move_counts", ctypes.POINTER(i64)), ("compress", i32),
                ("reserved", i32)]


class sp_exec_stats(ctypes.Structure):
    _fields_ = [("instances", i64), ("moved_in", i64), ("moved_out", i64), ("moves_hoisted", i64),
                ("max_levels", i32), ("smem_bytes", i32), ("ctas", i32), ("reserved", i32)]


class sp_tile_problem(ctypes.Structure):
    _fields_ = [("depth", i32), ("n_refs", i32), ("extent", ctypes.POINTER(i64)), ("refs", ctypes.POINTER(sp_ref)),
                ("n_cand", ctypes.POINTER(i32)), ("cand", ctypes.POINTER(i64)), ("mup_elems", i64), ("procs", i32),
                ("reserved", i32), ("sync_cost", f64), ("elem_cost", f64)]


class sp_tile_result(ctypes.Structure):
    _fields_ = [("tile", i64 * 8), ("cost", f64), ("local_elems", i64), ("evaluated", i64), ("feasible", i32),
                ("reserved", i32)]


SYMBOLS = {
    "sp_status_string": (ctypes.c_char_p, [ctypes.c_int]),
    "sp_last_cuda_error": (ctypes.c_int, []),
    "sp_last_nccl_error": (ctypes.c_int, []),
    "sp_version": (ctypes.c_int, []),
    "sp_abi_struct_sizes": (ctypes.c_int, [ctypes.POINTER(i64), i32]),
    "sp_plan_buffers": (ctypes.c_int, [ctypes.POINTER(sp_block), ctypes.POINTER(sp_plan_opts), ctypes.POINTER(sp_buffer),
                                       i32, ctypes.POINTER(i32), ctypes.POINTER(i32), ctypes.POINTER(i64)]),
    "sp_jacobi1d_plan": (ctypes.c_int, [i64, i32, i32, i32, ctypes.POINTER(sp_jacobi_plan)]),
    "sp_jacobi1d_tile_footprint": (ctypes.c_int, [i64, i32, i64, i64, ctypes.POINTER(i64), ctypes.POINTER(i64)]),
    "sp_jacobi1d_timetiled": (ctypes.c_int, [vp, vp, i64, i32, i32, i32, vp, vp]),
    "sp_jacobi1d_pass_segment": (ctypes.c_int, [vp, vp, i64, i64, i64, i64, i64, i32, i32, i32, vp]),
    "sp_jacobi1d_timetiled_fused": (ctypes.c_int, [vp, vp, vp, i64, i64, i32, i32, i32, vp, vp]),
    "sp_jacobi1d_timetiled_stream": (ctypes.c_int, [vp, vp, vp, vp, vp, i64, i64, i32, i32, i32, i64, vp, vp]),
    "sp_jacobi1d_host": (ctypes.c_int, [vp, vp, vp, vp, i64, i64, i32, i32, i32, vp]),
    "sp_jacobi1d_host_flags_len": (ctypes.c_int, [i64, i32, i32, i32, ctypes.POINTER(i64)]),
    "sp_jacobi1d_resident_capacity": (ctypes.c_int, [ctypes.POINTER(i64)]),
    "sp_jacobi1d_resident": (ctypes.c_int, [vp, vp, i64, i32, vp]),
    "sp_me_sad_search": (ctypes.c_int, [vp, vp, i64, i32, i32, i32, i32, i32, i64, i32, i32, i32, i32, vp, vp, vp, vp]),
    "sp_me_sad_search_range": (ctypes.c_int, [vp, vp, i64, i32, i32, i32, i64, i32, i32, i64, i64, vp, vp, vp]),
    "sp_me_sad_search_gather": (ctypes.c_int, [ctypes.POINTER(sp_me_gather_links), vp, vp, i64, i32, i32, i32, i64, i32,
                                               i32, i64, i64, vp]),
    "sp_me_sad_search_dist": (ctypes.c_int, [vp, vp, vp, i64, i32, i32, i32, i64, i32, i32, ctypes.POINTER(i64), vp, vp,
                                             vp]),
    "sp_me_search_host": (ctypes.c_int, [vp, i64, i32, i32, i32, i32, vp, vp, vp, vp, vp, vp]),
    "sp_me_ref_window": (ctypes.c_int, [i32, i32, i32, i32, i32, ctypes.POINTER(i64), ctypes.POINTER(i64)]),
    "sp_get_unique_id": (ctypes.c_int, [ctypes.POINTER(ctypes.c_uint8)]),
    "sp_comm_init": (ctypes.c_int, [ctypes.POINTER(vp), ctypes.POINTER(ctypes.c_uint8), i32, i32, i32]),
    "sp_comm_destroy": (ctypes.c_int, [vp]),
    "sp_jacobi1d_timetiled_dist": (ctypes.c_int, [vp, vp, vp, i64, i64, i64, i32, i32, i32, vp]),
    "sp_jacobi1d_timetiled_loopback": (ctypes.c_int, [ctypes.POINTER(vp), ctypes.POINTER(vp), i32, i64,
                                                      ctypes.POINTER(i64), ctypes.POINTER(i64), i32, i32, i32, vp]),
    "sp_allgather": (ctypes.c_int, [vp, vp, vp, i64, vp]),
    "sp_comm_async_error": (ctypes.c_int, [vp, ctypes.POINTER(i32)]),
    "sp_comm_sync": (ctypes.c_int, [vp, vp, i64]),
    "sp_jacobi1d_untiled": (ctypes.c_int, [vp, vp, i64, i32, vp]),
    "sp_tile_search": (ctypes.c_int, [ctypes.POINTER(sp_tile_problem), ctypes.POINTER(sp_tile_result)]),
    "sp_me_sad_search_unrestricted": (ctypes.c_int, [vp, vp, i64, i32, i32, i32, i32, i64, i32, i32, vp, vp, vp, vp]),
    "sp_me_pad_frames": (ctypes.c_int, [vp, i64, i64, i32, i32, i32, i32, vp, i64, i64, vp]),
    "sp_jacobi1d_timetiled_peer": (ctypes.c_int, [ctypes.POINTER(sp_peer_links), vp, vp, i64, i64, i64, i32, i32, i32,
                                                  vp]),
    "sp_jacobi1d_timetiled_peer_fused": (ctypes.c_int, [ctypes.POINTER(sp_peer_links), vp, vp, vp, i64, i64, i64, i64,
                                                        i32, i32, i32, vp]),
    "sp_device_alloc": (ctypes.c_int, [ctypes.POINTER(vp), i64]),
    "sp_device_free": (ctypes.c_int, [vp]),
    "sp_ipc_get_handle": (ctypes.c_int, [vp, ctypes.POINTER(ctypes.c_uint8)]),
    "sp_ipc_open_handle": (ctypes.c_int, [ctypes.POINTER(ctypes.c_uint8), ctypes.POINTER(vp)]),
    "sp_ipc_close_handle": (ctypes.c_int, [vp]),
    "sp_me_sad_search_direct": (ctypes.c_int, [vp, vp, i64, i32, i32, i32, i32, i32, i64, i32, i32, i32, i32, vp, vp,
                                               vp, vp]),
    "sp_exec_block": (ctypes.c_int, [ctypes.POINTER(sp_block), ctypes.POINTER(sp_stmt_body), ctypes.POINTER(sp_array_desc),
                                     i32, ctypes.POINTER(sp_exec_opts), ctypes.POINTER(sp_exec_stats), vp]),
}


def _load():
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"libsp.so is not built ({LIB_PATH}); run `python -c 'import __graft_entry__ as g; g.build()'`."
                          " There is no CPU fallback.")
    L = ctypes.CDLL(LIB_PATH)
    for name, (res, args) in SYMBOLS.items():
        if os.environ.get("SP_LIB") and not hasattr(L, name):
            continue  # an experimental build (SP_LIB) may predate a symbol; the product lib may not
        fn = getattr(L, name)
        fn.restype = res
        fn.argtypes = args
    return L


lib = _load()


class SPError(RuntimeError):
    def __init__(self, status: int, where: str):
        self.status = status
        name = lib.sp_status_string(status).decode()
        extra = ""
        if name == "SP_ERR_CUDA":
            extra = f" (cudaError {lib.sp_last_cuda_error()})"
        elif name == "SP_ERR_NCCL":
            extra = f" (ncclResult {lib.sp_last_nccl_error()})"
        super().__init__(f"{where}: {name}{extra}")


def _check(status: int, where: str) -> None:
    if status != 0:
        raise SPError(status, where)


def _stream(stream):
    import torch
    if stream is None:
        return vp(torch.cuda.current_stream().cuda_stream)
    if isinstance(stream, int):
        return vp(stream)
    return vp(stream.cuda_stream)


def _ptr(t):
    return vp(t.data_ptr()) if t is not None else None


def _scratch(shape, dtype, device, stream):
    """Library scratch allocated for one call.  When the call runs on a stream other than the
    current one, the caching allocator is told so (record_stream): the block is then not handed
    out again before the work queued on that stream has finished with it."""
    import torch
    t = torch.empty(shape, dtype=dtype, device=device)
    if stream is not None and not isinstance(stream, int):
        t.record_stream(stream)
    elif isinstance(stream, int):
        t.record_stream(torch.cuda.ExternalStream(stream, device=t.device))
    return t


def halo_of(time_tile: int) -> int:
    return (int(time_tile) + 3) & ~3


# ---------------------------------------------------------------------------------------
# Planner
# ---------------------------------------------------------------------------------------
def _marshal_block(block: dict, P: int | None = None):
    """sp_block for {"params": [...], "stmts": [{"depth", "rows"}], "refs": [{"stmt", "array",
    "is_write", "rank", "rows"}]}; returns (blk, keepalive)."""
    params = [int(p) for p in block.get("params", [])]
    P = len(params) if P is None else P
    keep = []
    doms = (sp_domain * max(1, len(block["stmts"])))()
    for k, s in enumerate(block["stmts"]):
        d = int(s["depth"])
        rows = np.ascontiguousarray(np.asarray(s["rows"], dtype=np.int64).reshape(-1, d + P + 1))
        keep.append(rows)
        doms[k] = sp_domain(d, rows.shape[0], rows.ctypes.data_as(ctypes.POINTER(i64)))
    refs = (sp_ref * max(1, len(block["refs"])))()
    for k, r in enumerate(block["refs"]):
        rows = np.ascontiguousarray(np.asarray(r["rows"], dtype=np.int64))
        keep.append(rows)
        refs[k] = sp_ref(int(r["stmt"]), int(r["array"]), int(bool(r["is_write"])), int(r["rank"]),
                         rows.ctypes.data_as(ctypes.POINTER(i64)))
    par = np.ascontiguousarray(np.asarray(params if params else [0] * max(1, P), dtype=np.int64))
    keep += [doms, refs, par]
    blk = sp_block(P, len(block["stmts"]), len(block["refs"]), 0, par.ctypes.data_as(ctypes.POINTER(i64)), doms, refs)
    return blk, keep


def plan_buffers(block: dict, mode: int = PER_ARRAY, delta: float = 0.30, reuse_filter: bool = False,
                 mup_elems: int = 0, max_points: int = 0, cap: int = 64, compress: bool = False) -> dict:
    """sp_plan_buffers on a block given as {"params": [...], "stmts": [{"depth", "rows"}],
    "refs": [{"stmt", "array", "is_write", "rank", "rows"}]} (extra keys ignored)."""
    params = [int(p) for p in block.get("params", [])]
    P = len(params)
    blk, keep = _marshal_block(block)
    opts = sp_plan_opts(int(mode), int(bool(reuse_filter)), float(delta), int(mup_elems), int(max_points),
                        int(bool(compress)), 0)
    n_refs = len(block["refs"])
    ref_buf = (i32 * max(1, n_refs))()
    width = sum(int(r["rank"]) * (int(block["stmts"][int(r["stmt"])]["depth"]) + P + 1) for r in block["refs"])
    local = (i64 * max(1, width))()
    n = i32(0)
    while True:
        bufs = (sp_buffer * cap)()
        st = lib.sp_plan_buffers(ctypes.byref(blk), ctypes.byref(opts), bufs, cap, ctypes.byref(n), ref_buf, local)
        if st == -3 and n.value > cap:  # SP_ERR_CAPACITY: retry with the required count
            cap = n.value
            continue
        break
    out = {"status": st, "buffers": [], "ref_buf": [], "local_rows": []}
    if st not in (0, -6):
        return out
    for b in bufs[: n.value]:
        rk = b.rank
        out["buffers"].append({
            "array": b.array, "rank": rk, "beneficial": b.beneficial, "n_refs": b.n_refs,
            "lb": list(b.lb[:rk]), "ub": list(b.ub[:rk]), "size": b.size, "v_in_ub": b.v_in_ub, "v_out_ub": b.v_out_ub,
            "in_lb": list(b.in_lb[:rk]), "in_ub": list(b.in_ub[:rk]), "in_count": b.in_count, "in_dense": b.in_dense,
            "out_lb": list(b.out_lb[:rk]), "out_ub": list(b.out_ub[:rk]), "out_count": b.out_count,
            "out_dense": b.out_dense, "overlap": b.overlap, "union_count": b.union_count,
            "n_dims": b.n_dims, "kept": [k for k in range(rk) if (b.kept_mask >> k) & 1],
        })
    if st != 0:
        return out
    out["ref_buf"] = list(ref_buf[:n_refs])
    pos = 0
    for r in block["refs"]:
        w = int(block["stmts"][int(r["stmt"])]["depth"]) + P + 1
        rk = int(r["rank"])
        out["local_rows"].append([list(local[pos + k * w: pos + (k + 1) * w]) for k in range(rk)])
        pos += rk * w
    return out


OP_LOAD, OP_CONST, OP_ADD, OP_SUB, OP_MUL = 0, 1, 2, 3, 4
_OPS = {"load": OP_LOAD, "const": OP_CONST, "add": OP_ADD, "sub": OP_SUB, "mul": OP_MUL}


MOVE_ALL, MOVE_DATAFLOW = 0, 1


def exec_block(block: dict, bodies: list, arrays: list, tile_params=None, tiles_per_cta: int = 1,
               hoist: bool = True, reuse_filter: bool = False, max_points: int = 0, movement: int = MOVE_ALL,
               live_out=None, dry_run: bool = False, compress: bool = False, stream=None) -> dict:
    """sp_exec_block (staged-tile executor).  arrays: CUDA float32 contiguous
    tensors indexed by array id (updated in place).  bodies[s] = {"write_ref": r, "beta": [...],
    "ops": [(op, arg), ...]} with op in OP_LOAD (arg = ref index), OP_CONST (arg = value),
    OP_ADD, OP_SUB, OP_MUL (arg ignored).  tile_params: [n_tiles][n_params] (None: one tile with
    block["params"]).  Returns the sp_exec_stats fields."""
    import torch
    P = len(block.get("params", [])) if tile_params is None else (len(tile_params[0]) if len(tile_params) else 0)
    blk, keep = _marshal_block(block, P)
    S = len(block["stmts"])
    bl = (sp_stmt_body * max(1, S))()
    for k, b in enumerate(bodies):
        ops = (sp_op * max(1, len(b["ops"])))()
        for q, (op, arg) in enumerate(b["ops"]):
            op = _OPS[op] if isinstance(op, str) else int(op)
            ops[q] = sp_op(op, int(arg) if op == OP_LOAD else 0, float(arg) if op == OP_CONST else 0.0, 0)
        beta = (i32 * (len(b["beta"])))(*[int(v) for v in b["beta"]])
        keep += [ops, beta]
        bl[k] = sp_stmt_body(int(b["write_ref"]), len(b["ops"]), ops, beta)
    ad = (sp_array_desc * len(arrays))()
    for k, a in enumerate(arrays):
        assert a.dtype == torch.float32 and a.is_contiguous() and (a.is_cuda or dry_run)
        ext = (i64 * 8)(*list(a.shape))
        ad[k] = sp_array_desc(a.data_ptr() if a.is_cuda else 16, a.dim(), 0, ext)
    if tile_params is None:
        tp, n_tiles = None, 1
    else:
        tparr = np.ascontiguousarray(np.asarray(tile_params, dtype=np.int64).reshape(len(tile_params), -1))
        keep.append(tparr)
        tp, n_tiles = tparr.ctypes.data_as(ctypes.POINTER(i64)), tparr.shape[0]
    lo = None if live_out is None else (i32 * len(arrays))(*[int(bool(v)) for v in live_out])
    counts = (i64 * (2 * n_tiles * len(arrays)))()
    opts = sp_exec_opts(n_tiles, int(tiles_per_cta), tp, int(bool(hoist)), int(bool(reuse_filter)), int(max_points),
                        int(movement), int(bool(dry_run)), lo, counts, int(bool(compress)), 0)
    stats = sp_exec_stats()
    _check(lib.sp_exec_block(ctypes.byref(blk), bl, ad, len(arrays), ctypes.byref(opts), ctypes.byref(stats),
                             None if dry_run else _stream(stream)), "sp_exec_block")
    out = {f: getattr(stats, f) for f, _ in sp_exec_stats._fields_ if f != "reserved"}
    out["move_counts"] = np.array(counts[:], dtype=np.int64).reshape(n_tiles, len(arrays), 2)
    return out


def tile_search(extent, refs, candidates, mup_elems: int = 0, procs: int = 32, sync_cost: float = 1.0,
                elem_cost: float = 1.0) -> dict:
    """sp_tile_search (§4.3).  extent: [m] trip counts; refs: [{"array", "is_write", "rank",
    "rows" [rank][m+1]}] over tile-local iterators; candidates: per loop, a list of sizes."""
    m = len(extent)
    ext = np.ascontiguousarray(np.asarray(extent, dtype=np.int64))
    keep = []
    rr = (sp_ref * len(refs))()
    for k, r in enumerate(refs):
        rows = np.ascontiguousarray(np.asarray(r["rows"], dtype=np.int64))
        keep.append(rows)
        rr[k] = sp_ref(0, int(r["array"]), int(bool(r["is_write"])), int(r["rank"]),
                       rows.ctypes.data_as(ctypes.POINTER(i64)))
    nc = (i32 * m)(*[len(c) for c in candidates])
    flat = np.ascontiguousarray(np.asarray([x for c in candidates for x in c], dtype=np.int64))
    prob = sp_tile_problem(m, len(refs), ext.ctypes.data_as(ctypes.POINTER(i64)), rr, nc,
                           flat.ctypes.data_as(ctypes.POINTER(i64)), int(mup_elems), int(procs), 0, float(sync_cost),
                           float(elem_cost))
    res = sp_tile_result()
    _check(lib.sp_tile_search(ctypes.byref(prob), ctypes.byref(res)), "sp_tile_search")
    return {"tile": list(res.tile[:m]), "cost": res.cost, "local_elems": res.local_elems, "evaluated": res.evaluated,
            "feasible": bool(res.feasible)}


# ---------------------------------------------------------------------------------------
# Jacobi
# ---------------------------------------------------------------------------------------
def jacobi1d_plan(n: int, steps: int, time_tile: int = 16, space_tile: int = 0) -> dict:
    p = sp_jacobi_plan()
    _check(lib.sp_jacobi1d_plan(int(n), int(steps), int(time_tile), int(space_tile), ctypes.byref(p)), "sp_jacobi1d_plan")
    return {f: getattr(p, f) for f, _ in sp_jacobi_plan._fields_}


def jacobi1d_tile_footprint(n: int, h: int, x0: int, space_tile: int) -> tuple[int, int]:
    lb, ub = i64(), i64()
    _check(lib.sp_jacobi1d_tile_footprint(int(n), int(h), int(x0), int(space_tile), ctypes.byref(lb), ctypes.byref(ub)),
           "sp_jacobi1d_tile_footprint")
    return lb.value, ub.value


def jacobi1d_timetiled(a, steps: int, time_tile: int = 16, space_tile: int = 0, work=None, footprint_log=None,
                       stream=None):
    """In place on a CUDA float32 tensor a[n]; work (same shape) is allocated if None."""
    import torch
    assert a.is_cuda and a.dtype == torch.float32 and a.is_contiguous()
    if work is None:
        work = _scratch(a.shape, a.dtype, a.device, stream)
    _check(lib.sp_jacobi1d_timetiled(_ptr(a), _ptr(work), a.numel(), int(steps), int(time_tile), int(space_tile),
                                     _ptr(footprint_log), _stream(stream)), "sp_jacobi1d_timetiled")
    return a


def jacobi1d_timetiled_fused(a, steps: int, time_tile: int = 64, space_tile: int = 0, work=None, flags=None,
                             footprint_log=None, stream=None):
    """All passes in one persistent launch (sp_jacobi1d_timetiled_fused).  flags: device int32
    scratch of >= plan["tiles"] + 1 entries (allocated if None)."""
    import torch
    assert a.is_cuda and a.dtype == torch.float32 and a.is_contiguous()
    if work is None:
        work = _scratch(a.shape, a.dtype, a.device, stream)
    if flags is None:
        flags = _scratch(jacobi1d_plan(a.numel(), steps, time_tile, space_tile)["tiles"] + 1, torch.int32, a.device,
                         stream)
    _check(lib.sp_jacobi1d_timetiled_fused(_ptr(a), _ptr(work), _ptr(flags), flags.numel(), a.numel(), int(steps),
                                           int(time_tile), int(space_tile), _ptr(footprint_log), _stream(stream)),
           "sp_jacobi1d_timetiled_fused")
    return a


def jacobi1d_timetiled_stream(inp, out, steps: int, time_tile: int = 64, space_tile: int = 0, skew: int = -1,
                              buf0=None, buf1=None, flags=None, footprint_log=None, stream=None):
    """out = J^steps(inp) in one persistent launch (sp_jacobi1d_timetiled_stream).  inp / out:
    CUDA or PINNED CPU float32 tensors (host memory is streamed by the kernel's TMA move-in /
    move-out); skew: 0 pass-major, D > 0 wavefront, < 0 library default."""
    import torch
    n = inp.numel()
    assert inp.dtype == torch.float32 and out.dtype == torch.float32 and out.numel() == n
    dev = inp.device if inp.is_cuda else (out.device if out.is_cuda else torch.device("cuda"))
    if buf0 is None:
        buf0 = _scratch(n, torch.float32, dev, stream)
    if buf1 is None:
        buf1 = _scratch(n, torch.float32, dev, stream)
    if flags is None:
        flags = _scratch(jacobi1d_plan(n, steps, time_tile, space_tile)["tiles"] + 1, torch.int32, dev, stream)
    _check(lib.sp_jacobi1d_timetiled_stream(_ptr(inp), _ptr(out), _ptr(buf0), _ptr(buf1), _ptr(flags), flags.numel(), n,
                                            int(steps), int(time_tile), int(space_tile), int(skew), _ptr(footprint_log),
                                            _stream(stream)), "sp_jacobi1d_timetiled_stream")
    return out


def jacobi1d_resident_capacity() -> int:
    c = i64()
    _check(lib.sp_jacobi1d_resident_capacity(ctypes.byref(c)), "sp_jacobi1d_resident_capacity")
    return c.value


def jacobi1d_resident(inp, steps: int, out=None, stream=None):
    """Small domains: out = J^steps(inp) in one thread-block cluster (sp_jacobi1d_resident);
    inp / out CUDA float32 (out defaults to inp, in place)."""
    import torch
    assert inp.is_cuda and inp.dtype == torch.float32 and inp.is_contiguous()
    out = inp if out is None else out
    _check(lib.sp_jacobi1d_resident(_ptr(inp), _ptr(out), inp.numel(), int(steps), _stream(stream)),
           "sp_jacobi1d_resident")
    return out


def jacobi1d_host_flags_len(n: int, steps: int, time_tile: int = 64, space_tile: int = 0) -> int:
    """flags length that selects sp_jacobi1d_host's copy-engine input (host-only)."""
    c = i64()
    _check(lib.sp_jacobi1d_host_flags_len(int(n), int(steps), int(time_tile), int(space_tile), ctypes.byref(c)),
           "sp_jacobi1d_host_flags_len")
    return c.value


class Jacobi1DHost:
    """Reusable device scratch for the end-to-end host-buffer call (sp_jacobi1d_host): two
    n-cell device buffers and the completion / input-ready flags, allocated once.
    direct_input=True sizes the flags for pass 0's own PCIe reads of the host array instead
    of the copy-engine input (the round-2 form; A/B and tests)."""

    def __init__(self, n: int, steps: int, time_tile: int = 64, space_tile: int = 0, device="cuda",
                 direct_input: bool = False):
        import torch
        self.n, self.steps, self.time_tile, self.space_tile = n, steps, time_tile, space_tile
        self.buf0 = torch.empty(n, dtype=torch.float32, device=device)
        self.buf1 = torch.empty(n, dtype=torch.float32, device=device)
        nf = (jacobi1d_plan(n, steps, time_tile, space_tile)["persistent_tiles"] + 1 if direct_input
              else jacobi1d_host_flags_len(n, steps, time_tile, space_tile))
        self.flags = torch.empty(nf, dtype=torch.int32, device=device)

    def run(self, a_pinned, stream=None):
        """In place on a PINNED CPU float32 tensor: a_pinned <- J^steps(a_pinned) (stream-ordered;
        synchronize before reading it)."""
        assert a_pinned.is_pinned() and a_pinned.numel() == self.n and a_pinned.is_contiguous()
        _check(lib.sp_jacobi1d_host(_ptr(a_pinned), _ptr(self.buf0), _ptr(self.buf1), _ptr(self.flags),
                                    self.flags.numel(), self.n, int(self.steps), int(self.time_tile),
                                    int(self.space_tile), _stream(stream)), "sp_jacobi1d_host")
        return a_pinned


def jacobi1d_untiled(a, steps: int, work=None, stream=None):
    """N1 ablation: no staging, no time tiling (one launch per step).  In place on a[n]."""
    import torch
    if work is None:
        work = _scratch(a.shape, a.dtype, a.device, stream)
    _check(lib.sp_jacobi1d_untiled(_ptr(a), _ptr(work), a.numel(), int(steps), _stream(stream)), "sp_jacobi1d_untiled")
    return a


def jacobi1d_pass_segment(src, dst, n_global: int, g0: int, own_begin: int, own_end: int, h: int, time_tile: int,
                          space_tile: int = 0, stream=None):
    _check(lib.sp_jacobi1d_pass_segment(_ptr(src), _ptr(dst), int(n_global), int(g0), src.numel(), int(own_begin),
                                        int(own_end), int(h), int(time_tile), int(space_tile), _stream(stream)),
           "sp_jacobi1d_pass_segment")


def jacobi1d_timetiled_loopback(a_locals, work_locals, n_global: int, x_begins, n_locals, steps: int,
                                time_tile: int = 16, space_tile: int = 0, stream=None):
    k = len(a_locals)
    A = (vp * k)(*[t.data_ptr() for t in a_locals])
    Wk = (vp * k)(*[t.data_ptr() for t in work_locals])
    xb = (i64 * k)(*[int(v) for v in x_begins])
    nl = (i64 * k)(*[int(v) for v in n_locals])
    _check(lib.sp_jacobi1d_timetiled_loopback(A, Wk, k, int(n_global), xb, nl, int(steps), int(time_tile),
                                              int(space_tile), _stream(stream)), "sp_jacobi1d_timetiled_loopback")


def jacobi1d(a_host, steps: int, time_tile: int = 64, space_tile: int = 0, device="cuda"):
    """End-to-end public call on a host array (numpy or CPU tensor): returns J^steps(a_host) as
    a pinned CPU tensor.  The input is copied into page-locked memory if it is not already
    there; the kernel then reads it and writes the result over PCIe itself (sp_jacobi1d_host)."""
    import torch
    h = torch.from_numpy(np.ascontiguousarray(a_host, dtype=np.float32)) if isinstance(a_host, np.ndarray) else a_host
    out = h.contiguous().pin_memory() if not h.is_pinned() else h.clone().pin_memory()
    Jacobi1DHost(out.numel(), steps, time_tile, space_tile, device).run(out)
    torch.cuda.synchronize(device)
    return out


# ---------------------------------------------------------------------------------------
# Motion estimation
# ---------------------------------------------------------------------------------------
def me_ref_window(width: int, frame_height: int, search_range: int, bx: int, by: int):
    lb, ub = (i64 * 2)(), (i64 * 2)()
    _check(lib.sp_me_ref_window(int(width), int(frame_height), int(search_range), int(bx), int(by), lb, ub),
           "sp_me_ref_window")
    return (lb[0], lb[1]), (ub[0], ub[1])


def me_sad_search(ref, cur, width: int, frame_height: int, search_range: int, *, row0: int = 0,
                  mb_row_begin: int = 0, mb_row_end: int | None = None, with_surface: bool = False,
                  out=None, stream=None):
    """ref, cur: CUDA uint8 tensors [n_pairs, rows_in_buffer, pitch] (views allowed, e.g.
    seq[0:64] and seq[1:65]); returns (mv [P, rows, mbx, 2] int16, sad [P, rows, mbx] uint32
    as int32 bits, surface or None)."""
    import torch
    assert ref.is_cuda and cur.is_cuda and ref.dtype == torch.uint8 and cur.dtype == torch.uint8
    assert ref.dim() == 3 and ref.shape == cur.shape and ref.stride() == cur.stride() and ref.stride(2) == 1
    n_pairs, rows_in_buffer, _ = ref.shape
    pitch = ref.stride(1)
    pair_stride = ref.stride(0) if n_pairs > 1 else pitch * rows_in_buffer
    mbx = width // 16
    if mb_row_end is None:
        mb_row_end = frame_height // 16
    rows = mb_row_end - mb_row_begin
    side = 2 * search_range + 1
    if out is None:
        mv = torch.empty((n_pairs, rows, mbx, 2), dtype=torch.int16, device=ref.device)
        sad = torch.empty((n_pairs, rows, mbx), dtype=torch.int32, device=ref.device)
        surf = torch.empty((n_pairs, rows, mbx, side * side), dtype=torch.int32, device=ref.device) if with_surface else None
    else:
        mv, sad, surf = out
    _check(lib.sp_me_sad_search(_ptr(ref), _ptr(cur), pitch, int(width), int(rows_in_buffer), int(row0),
                                int(frame_height), int(n_pairs), int(pair_stride), 16, int(search_range),
                                int(mb_row_begin), int(mb_row_end), _ptr(mv), _ptr(sad), _ptr(surf), _stream(stream)),
           "sp_me_sad_search")
    return mv, sad, surf


def me_sad_search_direct(ref, cur, width: int, frame_height: int, search_range: int, *, row0: int = 0,
                         mb_row_begin: int = 0, mb_row_end: int | None = None, with_surface: bool = False,
                         out=None, stream=None):
    """N1 ablation: same as me_sad_search, candidates read straight from global memory."""
    import torch
    n_pairs, rows_in_buffer, _ = ref.shape
    pitch = ref.stride(1)
    pair_stride = ref.stride(0) if n_pairs > 1 else pitch * rows_in_buffer
    mbx = width // 16
    if mb_row_end is None:
        mb_row_end = frame_height // 16
    rows = mb_row_end - mb_row_begin
    side = 2 * search_range + 1
    if out is None:
        mv = torch.empty((n_pairs, rows, mbx, 2), dtype=torch.int16, device=ref.device)
        sad = torch.empty((n_pairs, rows, mbx), dtype=torch.int32, device=ref.device)
        surf = torch.empty((n_pairs, rows, mbx, side * side), dtype=torch.int32, device=ref.device) if with_surface else None
    else:
        mv, sad, surf = out
    _check(lib.sp_me_sad_search_direct(_ptr(ref), _ptr(cur), pitch, int(width), int(rows_in_buffer), int(row0),
                                       int(frame_height), int(n_pairs), int(pair_stride), 16, int(search_range),
                                       int(mb_row_begin), int(mb_row_end), _ptr(mv), _ptr(sad), _ptr(surf),
                                       _stream(stream)), "sp_me_sad_search_direct")
    return mv, sad, surf


def me_pad_frames(frames, width: int, height: int, pad: int, stream=None):
    """Edge-extend a CUDA uint8 sequence [F, H, pitch] by `pad` pixels (sp_me_pad_frames);
    returns [F, H + 2 pad, P] with P = width + 2 pad rounded up to 16."""
    import torch
    F = frames.shape[0]
    P = (width + 2 * pad + 15) // 16 * 16
    out = torch.empty((F, height + 2 * pad, P), dtype=torch.uint8, device=frames.device)
    _check(lib.sp_me_pad_frames(_ptr(frames), frames.stride(1), frames.stride(0), int(width), int(height), F, int(pad),
                                _ptr(out), out.stride(1), out.stride(0), _stream(stream)), "sp_me_pad_frames")
    return out


def me_search_sequence_unrestricted(frames, width: int, height: int, search_range: int, with_surface: bool = False,
                                    stream=None):
    """Unrestricted-MV search (edge-extended reference) of the consecutive pairs of a CUDA
    uint8 sequence [F, H, pitch]: pads by max(R, 16) rounded to 16, then searches."""
    import torch
    pad = max(16, (int(search_range) + 15) // 16 * 16)
    padded = me_pad_frames(frames, width, height, pad, stream)
    ref, cur = padded[:-1], padded[1:]
    n_pairs = ref.shape[0]
    mbx, mby = width // 16, height // 16
    side = 2 * search_range + 1
    mv = torch.empty((n_pairs, mby, mbx, 2), dtype=torch.int16, device=frames.device)
    sad = torch.empty((n_pairs, mby, mbx), dtype=torch.int32, device=frames.device)
    surf = torch.empty((n_pairs, mby, mbx, side * side), dtype=torch.int32, device=frames.device) if with_surface else None
    _check(lib.sp_me_sad_search_unrestricted(_ptr(ref), _ptr(cur), ref.stride(1), int(width), int(height), pad, n_pairs,
                                             ref.stride(0), 16, int(search_range), _ptr(mv), _ptr(sad), _ptr(surf),
                                             _stream(stream)), "sp_me_sad_search_unrestricted")
    return mv, sad, surf


def me_search_sequence(frames, width: int, frame_height: int, search_range: int, **kw):
    """Pairs (ref = frame p, cur = frame p+1) of a CUDA uint8 sequence [F, H, pitch]."""
    return me_sad_search(frames[:-1], frames[1:], width, frame_height, search_range, **kw)


def me_sad_search_range(frames, width: int, frame_height: int, search_range: int, flat_begin: int, flat_end: int,
                        pair_base: int = 0, out=None, n_pairs_total: int | None = None, stream=None):
    """sp_me_sad_search_range: the macroblocks of flat (pair, MB row) rows [flat_begin, flat_end)
    of a batch.  frames: CUDA uint8 [F, H, pitch] holding frames pair_base .. pair_base + F - 1
    (pair p = (frame p, frame p + 1)); out = (mv [P, mby, mbx, 2] int16, sad [P, mby, mbx] int32)
    global arrays (allocated for n_pairs_total pairs if None); only the range's entries are written."""
    import torch
    assert frames.is_cuda and frames.dtype == torch.uint8 and frames.dim() == 3 and frames.stride(2) == 1
    mbx, mby = width // 16, frame_height // 16
    if out is None:
        P = n_pairs_total if n_pairs_total is not None else pair_base + frames.shape[0] - 1
        out = (torch.zeros((P, mby, mbx, 2), dtype=torch.int16, device=frames.device),
               torch.zeros((P, mby, mbx), dtype=torch.int32, device=frames.device))
    mv, sad = out
    ref, cur = frames[:-1], frames[1:]
    _check(lib.sp_me_sad_search_range(_ptr(ref), _ptr(cur), frames.stride(1), int(width), int(frame_height),
                                      ref.shape[0], frames.stride(0), int(pair_base), int(search_range), int(flat_begin),
                                      int(flat_end), _ptr(mv), _ptr(sad), _stream(stream)), "sp_me_sad_search_range")
    return mv, sad


class MEShard:
    """One rank's share of a sharded ME batch (SURVEY §8(e) ME row) with the all-gather fused
    into the search kernel over peer memory (sp_me_sad_search_gather).

    The batch's n_pairs x mby (pair, MB row) space is split by partition.me_row_ranges over the
    ranks of the default process group; this rank holds the frames of the pairs its range
    touches (`frames`, [F, H, pitch] uint8, frames pair_base .. pair_base + F - 1), of which only
    the rows `needed_rows(f)` are read (the current blocks plus the R-row reference halo,
    partition.me_band_rows).  Outputs mv / sad are libsp-owned, CUDA-IPC-exported global arrays
    [n_pairs, mby, mbx](, 2) on every rank; after run() (stream-ordered) every rank's arrays
    hold the whole batch's results.  Handles are exchanged through torch.distributed (any
    backend); the data path uses no collective library."""

    def __init__(self, n_pairs: int, width: int, height: int, search_range: int, pitch: int | None = None):
        import torch
        import torch.distributed as dist
        from . import partition
        self.n_pairs, self.width, self.height, self.range = int(n_pairs), int(width), int(height), int(search_range)
        self.pitch = int(pitch) if pitch else (self.width + 15) // 16 * 16
        self.rank, self.world = dist.get_rank(), dist.get_world_size()
        if self.world > ME_MAX_RANKS:
            raise ValueError(f"at most {ME_MAX_RANKS} ranks")
        self.mbx, self.mby = self.width // 16, self.height // 16
        self.ranges = partition.me_row_ranges(self.n_pairs, self.height, self.range, self.world)
        self.flat_begin, self.flat_end = self.ranges[self.rank]
        self.pieces = partition.split_flat_range(self.flat_begin, self.flat_end, self.mby)
        if self.pieces:
            self.pair_base = self.pieces[0][0]
            n_frames = self.pieces[-1][0] - self.pair_base + 2
        else:
            self.pair_base, n_frames = 0, 2
        self.frames = torch.zeros((n_frames, self.height, self.pitch), dtype=torch.uint8, device="cuda")
        cells = self.n_pairs * self.mby * self.mbx
        self._own = []
        ptrs = []
        for nbytes in (4 * cells, 4 * cells, 16 * self.world):
            p = vp()
            _check(lib.sp_device_alloc(ctypes.byref(p), max(16, nbytes)), "sp_device_alloc")
            self._own.append(p.value)
            ptrs.append(p.value)
        self.mv_ptr, self.sad_ptr, self.flags_ptr = ptrs
        handles = []
        for q in ptrs:
            h = (ctypes.c_uint8 * 64)()
            _check(lib.sp_ipc_get_handle(vp(q), h), "sp_ipc_get_handle")
            handles.append(bytes(h))
        info = [None] * self.world
        dist.all_gather_object(info, handles)
        L = sp_me_gather_links()
        L.nranks, L.rank, L.epoch = self.world, self.rank, 0
        self._mapped = []
        for q in range(self.world):
            if q == self.rank:
                L.mv[q], L.sad[q], L.flags[q] = self.mv_ptr, self.sad_ptr, self.flags_ptr
                continue
            got = []
            for hb in info[q]:
                m = vp()
                _check(lib.sp_ipc_open_handle((ctypes.c_uint8 * 64)(*hb), ctypes.byref(m)), "sp_ipc_open_handle")
                self._mapped.append(m.value)
                got.append(m.value)
            L.mv[q], L.sad[q], L.flags[q] = got
        self.links = L
        self.mv = torch.as_tensor(_DevView(self.mv_ptr, cells * 2, "<i2"), device="cuda").view(
            self.n_pairs, self.mby, self.mbx, 2)
        self.sad = torch.as_tensor(_DevView(self.sad_ptr, cells, "<i4"), device="cuda").view(
            self.n_pairs, self.mby, self.mbx)
        dist.barrier()

    def needed_rows(self, f: int) -> list[tuple[int, int]]:
        """Rows of global frame f this rank's range reads, as disjoint intervals [r0, r1): as the
        reference of pair f (band rows with the R-row halo) and as the current frame of pair f - 1."""
        from . import partition
        return partition.me_needed_rows(self.pieces, f, self.height, self.range)

    def load_frames(self, frame_fn):
        """Fill the needed rows of this rank's frames from frame_fn(f) -> host uint8 [H, >= W]."""
        import torch
        for k in range(self.frames.shape[0]):
            f = self.pair_base + k
            bands = self.needed_rows(f)
            if bands:
                full = np.asarray(frame_fn(f))
                for r0, r1 in bands:
                    fr = np.ascontiguousarray(full[r0:r1, : self.width])
                    self.frames[k, r0:r1, : self.width].copy_(torch.from_numpy(fr))

    def run(self, stream=None):
        """Search this rank's range; every rank's results land in every rank's mv / sad
        (stream-ordered: the stream waits for all ranks).  Returns (mv, sad)."""
        self.links.epoch += 1
        ref, cur = self.frames[:-1], self.frames[1:]
        _check(lib.sp_me_sad_search_gather(ctypes.byref(self.links), _ptr(ref), _ptr(cur), self.frames.stride(1),
                                           self.width, self.height, ref.shape[0], self.frames.stride(0),
                                           self.pair_base, self.range, self.flat_begin, self.flat_end,
                                           _stream(stream)), "sp_me_sad_search_gather")
        return self.mv, self.sad

    def close(self):
        import torch
        import torch.distributed as dist
        torch.cuda.synchronize()
        dist.barrier()
        for q in self._mapped:
            lib.sp_ipc_close_handle(vp(q))
        self._mapped = []
        dist.barrier()
        for q in self._own:
            lib.sp_device_free(vp(q))
        self._own = []


class Prepared:
    """A libsp call with its arguments marshalled once (ctypes objects, device pointers, the
    stream), for latency-bound configurations where Python-side argument conversion would
    otherwise dominate (J1, M2: a few microseconds of GPU work per call).  Calling it issues
    exactly the C entry point; the tensors it was prepared with must stay alive and unmoved."""

    def __init__(self, cfn, args, where: str, keep=()):
        self._f, self._a, self._w, self._keep = cfn, tuple(args), where, tuple(keep)

    def __call__(self):
        st = self._f(*self._a)
        if st:
            raise SPError(st, self._w)


def me_search_prepared(frames, width: int, frame_height: int, search_range: int, out=None, stream=None) -> Prepared:
    """sp_me_sad_search over the consecutive pairs of a CUDA uint8 sequence [F, H, pitch],
    prepared once (outputs allocated here unless given); call the result to run the search."""
    import torch
    ref, cur = frames[:-1], frames[1:]
    n_pairs, rows_in_buffer, _ = ref.shape
    pitch = ref.stride(1)
    pair_stride = ref.stride(0) if n_pairs > 1 else pitch * rows_in_buffer
    mbx, mby = width // 16, frame_height // 16
    if out is None:
        out = (torch.empty((n_pairs, mby, mbx, 2), dtype=torch.int16, device=frames.device),
               torch.empty((n_pairs, mby, mbx), dtype=torch.int32, device=frames.device))
    mv, sad = out[0], out[1]
    args = (vp(ref.data_ptr()), vp(cur.data_ptr()), i64(pitch), i32(width), i32(rows_in_buffer), i32(0),
            i32(frame_height), i32(n_pairs), i64(pair_stride), i32(16), i32(search_range), i32(0), i32(mby),
            vp(mv.data_ptr()), vp(sad.data_ptr()), None, _stream(stream))
    p = Prepared(lib.sp_me_sad_search, args, "sp_me_sad_search", keep=(frames, mv, sad))
    p.mv, p.sad = mv, sad
    return p


def jacobi1d_resident_prepared(inp, steps: int, out=None, stream=None) -> Prepared:
    """sp_jacobi1d_resident prepared once (small domains: one thread-block cluster)."""
    out = inp if out is None else out
    args = (vp(inp.data_ptr()), vp(out.data_ptr()), i64(inp.numel()), i32(steps), _stream(stream))
    p = Prepared(lib.sp_jacobi1d_resident, args, "sp_jacobi1d_resident", keep=(inp, out))
    p.out = out
    return p


class MESearchHost:
    """Reusable device staging for the end-to-end host-buffer search (sp_me_search_host): the
    frame buffer and ready flags on the device, the outputs in pinned host memory (the kernel
    stores them over PCIe), and a copy stream — allocated once."""

    def __init__(self, n_frames: int, width: int, height: int, pitch: int, search_range: int, device="cuda"):
        import torch
        self.n_frames, self.width, self.height, self.pitch, self.range = n_frames, width, height, pitch, search_range
        self.frames_dev = torch.empty((n_frames, height, pitch), dtype=torch.uint8, device=device)
        self.ready = torch.empty(max(1, n_frames - 1), dtype=torch.int32, device=device)
        mbx, mby = width // 16, height // 16
        self.mv = torch.empty((max(0, n_frames - 1), mby, mbx, 2), dtype=torch.int16).pin_memory()
        self.sad = torch.empty((max(0, n_frames - 1), mby, mbx), dtype=torch.int32).pin_memory()
        self.copy_stream = torch.cuda.Stream(device=device)

    def run(self, frames_pinned, stream=None):
        """frames_pinned: PINNED uint8 tensor [n_frames, height, pitch]; returns (mv, sad) pinned
        CPU tensors, valid after the stream synchronizes."""
        assert frames_pinned.is_pinned() and tuple(frames_pinned.shape) == (self.n_frames, self.height, self.pitch)
        _check(lib.sp_me_search_host(_ptr(frames_pinned), self.pitch, self.width, self.height, self.n_frames,
                                     self.range, _ptr(self.frames_dev), _ptr(self.ready), _ptr(self.mv), _ptr(self.sad),
                                     _stream(stream), _stream(self.copy_stream)), "sp_me_search_host")
        return self.mv, self.sad


def me_search(frames_host, width: int, frame_height: int, search_range: int, device="cuda"):
    """End-to-end public call on a host frame sequence [F, H, pitch] (numpy or CPU tensor):
    frame-by-frame H2D copies overlapped with the search (sp_me_search_host; R in {16, 32}),
    MV / SAD stored into pinned host memory by the kernel.  Returns (mv, sad) CPU tensors."""
    import torch
    h = torch.from_numpy(np.ascontiguousarray(frames_host)) if isinstance(frames_host, np.ndarray) else frames_host
    if not h.is_pinned():
        h = h.contiguous().pin_memory()
    F, H, pitch = h.shape
    ctx = MESearchHost(F, width, frame_height, pitch, search_range, device)
    mv, sad = ctx.run(h)
    torch.cuda.synchronize(device)
    return mv, sad


# ---------------------------------------------------------------------------------------
# Multi-GPU
# ---------------------------------------------------------------------------------------
def _nccl_path():
    try:
        import nvidia.nccl
        d = os.path.join(list(nvidia.nccl.__path__)[0], "lib", "libnccl.so.2")
        return d if os.path.exists(d) else None
    except Exception:
        return None


def get_unique_id() -> bytes:
    if "SP_NCCL_LIB" not in os.environ and _nccl_path():
        os.environ["SP_NCCL_LIB"] = _nccl_path()
    buf = (ctypes.c_uint8 * 128)()
    _check(lib.sp_get_unique_id(buf), "sp_get_unique_id")
    return bytes(buf)


class Comm:
    """NCCL communicator owned by libsp (one per process / GPU)."""

    def __init__(self, uid: bytes, nranks: int, rank: int, device: int):
        if "SP_NCCL_LIB" not in os.environ and _nccl_path():
            os.environ["SP_NCCL_LIB"] = _nccl_path()
        h = vp()
        buf = (ctypes.c_uint8 * 128)(*uid)
        _check(lib.sp_comm_init(ctypes.byref(h), buf, int(nranks), int(rank), int(device)), "sp_comm_init")
        self.handle = h
        self.nranks, self.rank, self.device = nranks, rank, device

    def destroy(self):
        if self.handle:
            _check(lib.sp_comm_destroy(self.handle), "sp_comm_destroy")
            self.handle = None

    def jacobi1d_timetiled_dist(self, a_local, work_local, n_global: int, x_begin: int, n_local: int, steps: int,
                                time_tile: int = 16, space_tile: int = 0, stream=None):
        _check(lib.sp_jacobi1d_timetiled_dist(self.handle, _ptr(a_local), _ptr(work_local), int(n_global), int(x_begin),
                                              int(n_local), int(steps), int(time_tile), int(space_tile),
                                              _stream(stream)), "sp_jacobi1d_timetiled_dist")

    def allgather(self, send, recv, stream=None):
        nbytes = send.numel() * send.element_size()
        _check(lib.sp_allgather(self.handle, _ptr(send), _ptr(recv), nbytes, _stream(stream)), "sp_allgather")

    def me_sad_search_dist(self, frames, width: int, frame_height: int, search_range: int, ranges, pair_base: int,
                           mv, sad, stream=None):
        """NCCL baseline of MEShard.run: this rank's range (ranges[rank]) searched into the
        global mv / sad, then grouped ncclBroadcasts (every rank roots its range)."""
        ref, cur = frames[:-1], frames[1:]
        fr = (i64 * (2 * len(ranges)))(*[int(v) for r in ranges for v in r])
        _check(lib.sp_me_sad_search_dist(self.handle, _ptr(ref), _ptr(cur), frames.stride(1), int(width),
                                         int(frame_height), ref.shape[0], frames.stride(0), int(pair_base),
                                         int(search_range), fr, _ptr(mv), _ptr(sad), _stream(stream)),
               "sp_me_sad_search_dist")
        return mv, sad

    def sync(self, timeout_ms: int = 60000, stream=None):
        """Wait for the stream with a deadline (sp_comm_sync): raises SPError(SP_ERR_NCCL) and
        aborts the communicator on an NCCL failure or when the deadline passes."""
        _check(lib.sp_comm_sync(self.handle, _stream(stream), int(timeout_ms)), "sp_comm_sync")

    def async_error(self) -> int:
        """ncclCommGetAsyncError of this communicator (0 = healthy, 7 = in progress)."""
        r = i32(0)
        _check(lib.sp_comm_async_error(self.handle, ctypes.byref(r)), "sp_comm_async_error")
        return r.value


# ---------------------------------------------------------------------------------------
# Fused peer-memory halo exchange (sp_jacobi1d_timetiled_peer)
# ---------------------------------------------------------------------------------------
class _DevView:
    """__cuda_array_interface__ view of a libsp device allocation (for torch.as_tensor)."""

    def __init__(self, ptr: int, n: int, typestr: str):
        self.__cuda_array_interface__ = {"shape": (n,), "typestr": typestr, "data": (ptr, False), "version": 3}


class PeerSlab:
    """One rank's slab of the distributed Jacobi domain for the fused peer-memory path.

    a / work / flags are CUDA-IPC-exportable allocations owned by libsp; the handles are
    exchanged with the neighbours through torch.distributed (any backend) and mapped, so the
    pass kernel stores halos straight into the neighbours' buffers (NVLink peer writes between
    GPUs; the same code runs between processes sharing one GPU).  `a` is a torch view of the
    rank's [x_begin - H, x_end + H) buffer."""

    def __init__(self, n_global: int, x_begin: int, n_local: int, time_tile: int, space_tile: int = 0,
                 fused: bool = False):
        """fused: one persistent launch per call with tile-granular halo exchange
        (sp_jacobi1d_timetiled_peer_fused); every rank of a run must pass the same value."""
        import torch
        import torch.distributed as dist
        self.n_global, self.x_begin, self.n_local = int(n_global), int(x_begin), int(n_local)
        self.time_tile, self.space_tile, self.fused = int(time_tile), int(space_tile), bool(fused)
        self._flags = None
        self.H = halo_of(time_tile)
        cells = self.n_local + 2 * self.H
        self._own = []
        ptrs = []
        for nbytes in (4 * cells, 4 * cells, 64):
            p = vp()
            _check(lib.sp_device_alloc(ctypes.byref(p), nbytes), "sp_device_alloc")
            self._own.append(p.value)
            ptrs.append(p.value)
        self.a_ptr, self.w_ptr, self.f_ptr = ptrs
        handles = []
        for p in ptrs:
            h = (ctypes.c_uint8 * 64)()
            _check(lib.sp_ipc_get_handle(vp(p), h), "sp_ipc_get_handle")
            handles.append(bytes(h))
        rank, world = dist.get_rank(), dist.get_world_size()
        info = [None] * world
        dist.all_gather_object(info, {"handles": handles, "n_local": self.n_local, "x_begin": self.x_begin})
        self._mapped = []

        def open_all(r):
            out = []
            for hb in info[r]["handles"]:
                q = vp()
                _check(lib.sp_ipc_open_handle((ctypes.c_uint8 * 64)(*hb), ctypes.byref(q)), "sp_ipc_open_handle")
                self._mapped.append(q.value)
                out.append(q.value)
            return out
        L = sp_peer_links()
        if self.x_begin > 0:
            la, lw, lf = open_all(rank - 1)
            L.left_bufs[0], L.left_bufs[1], L.left_flags = la, lw, lf
            L.left_n_local = info[rank - 1]["n_local"]
        if self.x_begin + self.n_local < self.n_global:
            ra, rw, rf = open_all(rank + 1)
            L.right_bufs[0], L.right_bufs[1], L.right_flags = ra, rw, rf
            L.right_n_local = info[rank + 1]["n_local"]
        L.my_flags = self.f_ptr
        L.epoch0 = 0
        self.links = L
        self.a = torch.as_tensor(_DevView(self.a_ptr, cells, "<f4"), device="cuda")
        self.work = torch.as_tensor(_DevView(self.w_ptr, cells, "<f4"), device="cuda")
        dist.barrier()

    def run(self, steps: int, stream=None):
        """sp_jacobi1d_timetiled_peer(_fused) over this slab; advances the epoch base."""
        import torch
        passes = (int(steps) + self.time_tile - 1) // self.time_tile
        if self.fused:
            tiles = jacobi1d_plan(self.n_local, max(1, int(steps)), self.time_tile, self.space_tile)["tiles"]
            need = tiles + 1 + 2 * passes
            if self._flags is None or self._flags.numel() < need:
                if self._flags is not None and stream is not None:  # the old block may still be in use there
                    self._flags.record_stream(stream if not isinstance(stream, int) else torch.cuda.ExternalStream(stream))
                self._flags = torch.empty(need, dtype=torch.int32, device="cuda")
            _check(lib.sp_jacobi1d_timetiled_peer_fused(ctypes.byref(self.links), vp(self.a_ptr), vp(self.w_ptr),
                                                        _ptr(self._flags), self._flags.numel(), self.n_global,
                                                        self.x_begin, self.n_local, int(steps), self.time_tile,
                                                        self.space_tile, _stream(stream)),
                   "sp_jacobi1d_timetiled_peer_fused")
        else:
            _check(lib.sp_jacobi1d_timetiled_peer(ctypes.byref(self.links), vp(self.a_ptr), vp(self.w_ptr),
                                                  self.n_global, self.x_begin, self.n_local, int(steps),
                                                  self.time_tile, self.space_tile, _stream(stream)),
                   "sp_jacobi1d_timetiled_peer")
        self.links.epoch0 += passes

    def close(self):
        import torch
        import torch.distributed as dist
        torch.cuda.synchronize()
        dist.barrier()
        for p in self._mapped:
            lib.sp_ipc_close_handle(vp(p))
        self._mapped = []
        dist.barrier()
        for p in self._own:
            lib.sp_device_free(vp(p))
        self._own = []
