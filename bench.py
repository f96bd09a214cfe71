"""Benchmark of the staged multi-level-tiled hot path (Baskaran et al., PPoPP'08) on B200.

One step = one pass of the whole hot path over one batch:
  * N = 1 (BASELINE configs 3 + 4):
      - Jacobi J3: T = 1024 steps of the fp32 1-D Jacobi stencil over 2^26 cells, time-tiled,
        every pass in one persistent launch with per-tile dependence flags;
      - ME M4: full-search SAD motion estimation of a 64-pair batch of 1920x1080 uint8 frames,
        +-32, 16x16 macroblocks.
  * N > 1 (BASELINE configs 5 + 4, strong scaling: the total problem is fixed):
      - Jacobi J5: 2^30 cells, T = 4096, split into N contiguous slabs; the halo exchange
        once per time tile is fused into each rank's persistent kernel as peer-memory stores
        over NVLink (default) or done by NCCL send/recv per pass (--halo nccl);
      - ME M4: the same 64-pair batch, its (pair, MB row) space split over the ranks by valid-
        candidate count; each rank holds only its band rows and the results are all-gathered
        by the search kernel itself over peer memory (default) or by grouped NCCL broadcasts
        (--gather nccl).
`value` = Jacobi point-updates of the whole job / max-over-ranks device time; ME's throughput
is reported in the `me` object with its own roofline.

  python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference] [--time-tile Tt]

With --gpus N > 1 and no torchrun environment, bench.py launches itself under
torch.distributed.run (one process per GPU, rendezvous on 127.0.0.1).
"""
from __future__ import annotations

import argparse
import json
import os
import socket
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "Jacobi GPoint-updates/s & ME SAD/s; %HBM roofline at 1/2/4/8 B200"
JAC3_N, JAC3_T = 1 << 26, 1024    # BASELINE config 3 (N = 1)
JAC5_N, JAC5_T = 1 << 30, 4096    # BASELINE config 5 (N > 1, strong scaling)
ME_W, ME_H, ME_R, ME_PAIRS = 1920, 1080, 32, 64
VABSDIFF4_PER_CLK_SM = 64  # measured issue rate (profiles/r01_ubench_issue_rates.txt)


def me_valid_sads(width, height, r, pairs, rows=None):
    """Valid 16x16 candidates (restricted vectors) of `pairs` pairs, or of the flat (pair, MB
    row) rows `rows` = (begin, end) of the batch."""
    mby = height // 16

    def row_count(by):
        y0 = 16 * by
        ny = min(r, height - 16 - y0) - max(-r, -y0) + 1
        return ny * sum(min(r, width - 16 - 16 * bx) - max(-r, -16 * bx) + 1 for bx in range(width // 16))
    per_row = [row_count(by) for by in range(mby)]
    if rows is None:
        return sum(per_row) * pairs
    return sum(per_row[k % mby] for k in range(rows[0], rows[1]))


def workload(world, tt):
    if world == 1:
        return {"name": "J3+M4", "jac_n": JAC3_N, "jac_t": JAC3_T}
    return {"name": "J5+M4", "jac_n": JAC5_N, "jac_t": JAC5_T}


def _geometry(n_local, T, tt, persistent):
    """The Jacobi pass kernel's geometry as the library plans it (include/sp.h sp_jacobi_plan):
    the persistent launches take the in-place one at Tt >= 48, the staged one otherwise."""
    import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
    pl = sp.jacobi1d_plan(n_local, T, tt, 0)
    if persistent and tt >= 48:
        k = (pl["persistent_space_tile"] + 2 * pl["halo"]) // 64  # strip = 64 K cells per warp
        return f"in place: {2 * k} cells/lane in {k + 1} packed registers, one stage per warp"
    return f"staged: {pl['cells_per_thread']} cells/lane, two stages per warp"


def bench_config(world, tt, halo="peer", gather="peer"):
    h = (tt + 3) & ~3
    if world == 1:
        return {"workload": f"J3: Jacobi fp32 N=2^26, T={JAC3_T}, time tile {tt} (halo {h}) + "
                            f"M4: ME {ME_W}x{ME_H} uint8 +-{ME_R}, {ME_PAIRS} pairs",
                "jacobi_global_n": JAC3_N, "jacobi_steps": JAC3_T, "time_tile": tt, "me_pairs_global": ME_PAIRS,
                "l2": "inputs larger than L2 (256 MiB Jacobi state, 135 MB frame batch); no flush",
                "parallelism": "1 GPU"}
    return {"workload": f"J5: Jacobi fp32 N=2^30, T={JAC5_T}, time tile {tt} (halo {h}), {world} slabs + "
                        f"M4: ME {ME_W}x{ME_H} uint8 +-{ME_R}, {ME_PAIRS} pairs sharded by MB rows",
            "jacobi_global_n": JAC5_N, "jacobi_steps": JAC5_T, "time_tile": tt, "me_pairs_global": ME_PAIRS,
            "l2": "inputs larger than L2 (4 GiB / N of Jacobi state per GPU); no flush",
            "parallelism": f"strong scaling over {world} GPUs; Jacobi halo exchange per time tile "
                           + ("fused into the persistent kernel (peer-memory stores over NVLink)" if halo == "peer"
                              else "by NCCL send/recv between per-pass launches")
                           + "; ME results all-gathered "
                           + ("by the search kernel (peer stores)" if gather == "peer" else "by NCCL broadcasts")}


def peaks():
    p = {"hbm_gbs": 6650.0, "sm_max_mhz": 1965.0, "source": "fallback (B200_PROFILING.md)"}
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            m = json.load(f)
        p = {"hbm_gbs": float(m["hbm_gbs"]), "sm_max_mhz": float(m.get("sm_max_mhz", 1965.0)),
             "source": "measured (MEASURED_PEAKS.json)"}
    except Exception:
        pass
    return p


class ClockSampler:
    """nvidia-smi clocks and throttle reasons sampled during the timed region."""

    def __init__(self, device: int):
        self.device = device
        self.proc = None
        self.lines: list[str] = []
        self.marks: list[float] = []

    def __enter__(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.device), "--query-gpu=timestamp,clocks.sm,clocks.max.sm,clocks_event_reasons.active,"
                 "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
                 "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap",
                 "--format=csv,noheader,nounits", "-lms", "100"],
                stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
            time.sleep(1.0)  # let nvidia-smi start sampling before the timed region
        except Exception:
            self.proc = None
        return self

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def __exit__(self, *a):
        if self.proc:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except Exception:
                self.proc.kill()
            self.t.join(timeout=2)

    def mark(self):
        self.marks.append(time.time())

    def summary(self):
        """Samples whose timestamp falls inside [first mark, last mark] (the timed region)."""
        import datetime
        sm, mx, reasons = [], None, set()
        lo = self.marks[0] if self.marks else 0.0
        hi = self.marks[-1] if self.marks else 1e30
        for ln in self.lines:
            f = [x.strip() for x in ln.split(",")]
            if len(f) < 8:
                continue
            try:
                ts = datetime.datetime.strptime(f[0], "%Y/%m/%d %H:%M:%S.%f").timestamp()
            except ValueError:
                continue
            if not (lo - 0.15 <= ts <= hi + 0.15):
                continue
            f = f[1:]
            try:
                sm.append(float(f[0]))
                mx = float(f[1])
            except ValueError:
                continue
            for name, v in zip(["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"], f[3:7]):
                if v.lower() == "active":
                    reasons.add(name)
        if not sm:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": [], "samples": 0}
        return {"sm_mhz": statistics.median(sm), "sm_max_mhz": mx, "reasons": sorted(reasons), "samples": len(sm)}


def traffic_from_profiles():
    """dram read+write bytes per launch from the committed ncu summary, if present."""
    try:
        with open(os.path.join(ROOT, "profiles", "ncu_traffic.json")) as f:
            return json.load(f)
    except Exception:
        return {}


# ---------------------------------------------------------------------------------------
# the CPU oracle, as it stands, on the host cores (reference arm and cpu_baseline)
# ---------------------------------------------------------------------------------------
def oracle_samples():
    """Bounded samples of the bench workload for the oracle: all host threads (~10-20 cpu-s)
    and one thread (~1 s)."""
    import oracle
    import sp_inputs
    cores = len(os.sched_getaffinity(0))
    a = sp_inputs.jacobi_input(JAC3_N, seed=sp_inputs.JACOBI_BENCH_SEED)
    fr0 = sp_inputs.me_frame(0, ME_W, ME_H, ME_R)
    fr1 = sp_inputs.me_frame(1, ME_W, ME_H, ME_R)
    mbx, mby = ME_W // 16, ME_H // 16
    out = {}
    for tag, threads, js, me_rows in (("all", cores, 32, (0, mby)), ("one", 1, 4, (30, 32))):
        oracle.set_threads(threads)
        t0 = time.perf_counter()
        oracle.jacobi1d(a, js)
        tj = time.perf_counter() - t0
        mbs = np.arange(me_rows[0] * mbx, me_rows[1] * mbx, dtype=np.int32)
        t0 = time.perf_counter()
        oracle.me_search(fr0, fr1, ME_W, ME_H, ME_R, mbs=mbs)
        tm = time.perf_counter() - t0
        out[tag] = {"jacobi_ups": (JAC3_N - 2) * js / tj, "me_sads": me_valid_sads(ME_W, ME_H, ME_R, 1, me_rows) / tm,
                    "threads": oracle.get_threads(), "jacobi_steps": js, "me_mb_rows": me_rows,
                    "seconds": tj + tm}
    oracle.set_threads(cores)
    a_ = out["all"]
    o_ = out["one"]
    return {"jacobi_ups": a_["jacobi_ups"], "me_sads": a_["me_sads"], "cores": a_["threads"],
            "jacobi_ups_1t": o_["jacobi_ups"], "me_sads_1t": o_["me_sads"], "cpu_model": oracle.cpu_model(),
            "sample": (f"all {a_['threads']} threads: Jacobi N=2^26 x {a_['jacobi_steps']} steps (of T=1024), "
                       f"ME one whole 1920x1080 pair at +-32 (M4 has 64); 1 thread: Jacobi N=2^26 x "
                       f"{o_['jacobi_steps']} steps, ME 2 interior MB rows"),
            "build": "gcc " + " ".join(oracle.CFLAGS)}


def cpu_baseline_obj(s, value_key="jacobi_ups"):
    return {"value": s[value_key] / 1e9, "unit": "GPoint-updates/s", "cores": s["cores"], "kind": "oracle",
            "sample": s["sample"], "value_1thread": s["jacobi_ups_1t"] / 1e9, "cpu_model": s["cpu_model"],
            "me_value": s["me_sads"] / 1e9, "me_value_1thread": s["me_sads_1t"] / 1e9, "me_unit": "GSAD/s",
            "build": s["build"]}


def run_reference(args, rank, world):
    if rank != 0:
        return 0
    for _ in range(args.warmup):
        oracle_samples()
    js, ms = [], []
    t_start = time.perf_counter()
    last = None
    for _ in range(args.steps):
        last = oracle_samples()
        js.append(last["jacobi_ups"])
        ms.append(last["me_sads"])
    tot = time.perf_counter() - t_start
    val = statistics.median(js) / 1e9
    cb = cpu_baseline_obj(last)
    cb["value"] = val
    line = {
        "impl": "reference", "metric": METRIC, "value": val, "unit": "GPoint-updates/s", "n_gpus": args.gpus,
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": tot / max(1, args.steps) * 1e3,
        "higher_is_better": True, "scaling": "weak" if args.gpus == 1 else "strong", "vs_baseline": None,
        "dtype": "f32/u8", "data": "synthetic",
        "config": dict(bench_config(args.gpus, args.time_tile),
                       note="oracle timed on bounded samples of the workload (see cpu_baseline.sample)"),
        "me": {"value": statistics.median(ms) / 1e9, "unit": "GSAD/s"},
        "cpu_baseline": cb,
        "e2e": {"value": val, "unit": "GPoint-updates/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


# ---------------------------------------------------------------------------------------
# our arm
# ---------------------------------------------------------------------------------------
def run_ours(args, rank, world, local_rank):
    import torch
    import torch.distributed as dist

    import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
    import sp_inputs
    from paper_conf_ppopp_baskaranbkrrs08_b200 import partition

    dev = torch.device("cuda", local_rank)
    torch.cuda.set_device(dev)
    stream = torch.cuda.current_stream()
    tt = args.time_tile
    H = sp.halo_of(tt)
    pk = peaks()
    wl = workload(world, tt)
    n_global, T = wl["jac_n"], wl["jac_t"]

    # ---- Jacobi state: this rank's slab [x_begin, x_begin + n_local) of the global domain
    x_begin, n_local = partition.jacobi_slabs(n_global, world, H)[rank]
    comm = None
    slab = None
    flags = None
    if world == 1:
        a_host = sp_inputs.jacobi_input(n_local, seed=sp_inputs.JACOBI_BENCH_SEED)
        a = torch.from_numpy(a_host).to(dev)
        work = torch.empty_like(a)
        # all passes in one persistent launch (per-tile completion flags + unit counter)
        flags = torch.empty(sp.jacobi1d_plan(n_local, T, tt, 0)["tiles"] + 1, dtype=torch.int32, device=dev)
    elif args.halo == "peer":
        # fused halo exchange: ONE persistent launch per step on every rank; the edge tiles
        # store their halos into the neighbours' buffers as soon as they complete
        slab = sp.PeerSlab(n_global, x_begin, n_local, tt, fused=True)
        slab.a[H:H + n_local] = torch.from_numpy(
            sp_inputs.jacobi_input(n_local, seed=sp_inputs.JACOBI_BENCH_SEED, begin=x_begin)).to(dev)
        a, work = slab.a, slab.work
    else:
        lo, hi = max(0, x_begin - H), min(n_global, x_begin + n_local + H)
        a = torch.zeros(n_local + 2 * H, dtype=torch.float32, device=dev)
        a[lo - (x_begin - H): hi - (x_begin - H)] = torch.from_numpy(
            sp_inputs.jacobi_input(hi - lo, seed=sp_inputs.JACOBI_BENCH_SEED, begin=lo)).to(dev)
        work = torch.empty_like(a)
    if world > 1 and (args.halo == "nccl" or args.gather == "nccl"):
        uid = [sp.get_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(uid, 0)
        comm = sp.Comm(uid[0], world, rank, local_rank)

    def jacobi_run(steps):
        if slab is not None:
            slab.run(steps)
        elif world > 1:
            comm.jacobi1d_timetiled_dist(a, work, n_global, x_begin, n_local, steps, tt, 0)
        else:
            sp.jacobi1d_timetiled_fused(a, steps, tt, 0, work=work, flags=flags)

    def jacobi_step():
        jacobi_run(T)

    # ---- ME batch: 64 pairs = frames [0, 65) of the sequence; N > 1: this rank's MB-row range
    mbx, mby = ME_W // 16, ME_H // 16
    me_shard = None
    frames_host = None
    if world == 1:
        frames_host = np.ascontiguousarray(np.stack([sp_inputs.me_frame(f, ME_W, ME_H, ME_R)
                                                     for f in range(ME_PAIRS + 1)]))
        frames = torch.from_numpy(frames_host).to(dev)
        me_out = (torch.empty((ME_PAIRS, mby, mbx, 2), dtype=torch.int16, device=dev),
                  torch.empty((ME_PAIRS, mby, mbx), dtype=torch.int32, device=dev), None)

        def me_step():
            sp.me_search_sequence(frames, ME_W, ME_H, ME_R, out=me_out)
    else:
        me_shard = sp.MEShard(ME_PAIRS, ME_W, ME_H, ME_R)
        me_shard.load_frames(lambda f: sp_inputs.me_frame(f, ME_W, ME_H, ME_R))
        if args.gather == "peer":
            def me_step():
                me_shard.run()
        else:
            def me_step():
                comm.me_sad_search_dist(me_shard.frames, ME_W, ME_H, ME_R, me_shard.ranges, me_shard.pair_base,
                                        me_shard.mv, me_shard.sad)

    def barrier():
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()

    # ---- timed region: K steps, device events on the launching stream.  The W warm-up steps
    # run inside the clock sampler's context, right before the timed region (the sampler's
    # start-up second would otherwise leave the GPU idle and its clocks ramping into step 1)
    K = args.steps
    ev = [[torch.cuda.Event(enable_timing=True) for _ in range(3)] for _ in range(K)]
    with ClockSampler(local_rank) as clk:
        for _ in range(args.warmup):
            jacobi_step()
            me_step()
        barrier()
        clk.mark()
        e_start = torch.cuda.Event(enable_timing=True)
        e_end = torch.cuda.Event(enable_timing=True)
        e_start.record(stream)
        for k in range(K):
            ev[k][0].record(stream)
            jacobi_step()
            ev[k][1].record(stream)
            me_step()
            ev[k][2].record(stream)
        e_end.record(stream)
        torch.cuda.synchronize()
        clk.mark()
        barrier()
    total_ms = e_start.elapsed_time(e_end)
    jac_steps = [ev[k][0].elapsed_time(ev[k][1]) for k in range(K)]
    me_steps = [ev[k][1].elapsed_time(ev[k][2]) for k in range(K)]
    jac_ms, me_ms = sum(jac_steps), sum(me_steps)
    # the median and the best step beside the mean (this rank's events)
    step_stats = {"jacobi_ms": {"median": round(float(np.median(jac_steps)), 4), "best": round(min(jac_steps), 4),
                                "steps": [round(x, 4) for x in jac_steps]},
                  "me_ms": {"median": round(float(np.median(me_steps)), 4), "best": round(min(me_steps), 4),
                            "steps": [round(x, 4) for x in me_steps]}}

    def max_over_ranks(x):
        if world == 1:
            return x
        t = torch.tensor([x], dtype=torch.float64, device="cpu" if dist.get_backend() == "gloo" else dev)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        return float(t.item())

    total_ms, jac_ms, me_ms = max_over_ranks(total_ms), max_over_ranks(jac_ms), max_over_ranks(me_ms)
    updates = (n_global - 2) * T * K
    sads = me_valid_sads(ME_W, ME_H, ME_R, ME_PAIRS) * K
    jac_val = updates / (jac_ms * 1e-3) / 1e9
    me_val = sads / (me_ms * 1e-3) / 1e9

    # ---- per-launch kernel durations (CUDA events on the launching stream) for the roofline
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    persistent = flags is not None or slab is not None
    if persistent:  # one persistent launch = all T steps
        reps, steps_per_launch = (3 if world == 1 else 1), T
        if world > 1:
            dist.barrier()
        e0.record(stream)
        for _ in range(reps):
            jacobi_run(T)
        e1.record(stream)
    else:  # one launch per pass (NCCL halo baseline): time full-height passes, exchange included
        reps, steps_per_launch = 4, tt
        if world > 1:
            dist.barrier()
        e0.record(stream)
        for _ in range(reps):
            jacobi_run(2 * tt)
        e1.record(stream)
        reps *= 2
    torch.cuda.synchronize()
    jac_launch_ms = e0.elapsed_time(e1) / reps
    jac_bytes = 8.0 * n_local * (steps_per_launch // tt)  # algorithmic: each cell read + written once per pass
    upd_local = n_local - (x_begin == 0) - (x_begin + n_local == n_global)  # this rank's updated cells
    jac_flops = 3.0 * upd_local * steps_per_launch  # algorithmic: 3 flops per point-update
    jac_gbs = jac_bytes / (jac_launch_ms * 1e-3) / 1e9
    jac_tflops = jac_flops / (jac_launch_ms * 1e-3) / 1e12
    fp32_peak = 148 * 128 * pk["sm_max_mhz"] * 1e6 / 1e12  # FADD/FMUL (and f32x2 forms) retire 128 flop/clk/SM
    if world > 1:
        dist.barrier()
    e0.record(stream)
    for _ in range(3):
        me_step()
    e1.record(stream)
    torch.cuda.synchronize()
    me_launch_ms = e0.elapsed_time(e1) / 3
    me_ops = (me_valid_sads(ME_W, ME_H, ME_R, ME_PAIRS) if world == 1 else
              me_valid_sads(ME_W, ME_H, ME_R, ME_PAIRS, (me_shard.flat_begin, me_shard.flat_end))) * 256.0
    me_achieved = me_ops / (me_launch_ms * 1e-3) / 1e12
    alu_peak = 148 * VABSDIFF4_PER_CLK_SM * 4 * pk["sm_max_mhz"] * 1e6 / 1e12
    tr = traffic_from_profiles()
    # Jacobi at Tt >= 16 is bound by the FP32 pipe (3 flops per update; HBM bytes per update
    # fall as 8/Tt): the binding roof is reported, with the HBM view beside it (north_star)
    kname = "jacobi1d_pass_kernel" + ("<kPeer>" if slab is not None else "")
    roof_jac = {"kernel": kname, "bound": "alu", "achieved": round(jac_tflops, 2),
                "peak": round(fp32_peak, 2), "unit": "TFLOP/s (fp32)", "frac": round(jac_tflops / fp32_peak, 4),
                "traffic": tr.get("jacobi1d_pass_kernel") if world == 1 else None,
                "peak_source": "148 SM x 128 fp32 lanes/clk x 1 op (the update is FADD, FADD, FMUL: no FMA to count twice; guide unit counts, microbenchmark-confirmed) x sm_max_mhz",
                "per_launch_ms": round(jac_launch_ms, 4), "algorithmic_flops_per_launch": jac_flops,
                "hbm": {"achieved": round(jac_gbs, 1), "peak": pk["hbm_gbs"], "unit": "GB/s",
                        "frac": round(jac_gbs / pk["hbm_gbs"], 4), "algorithmic_bytes_per_launch": jac_bytes,
                        "peak_source": pk["source"]}}
    roof_me = {"kernel": "me_sad_kernel" + ("<kGather>" if (me_shard is not None and args.gather == "peer") else ""),
               "bound": "alu", "achieved": round(me_achieved, 2), "peak": round(alu_peak, 2),
               "unit": "Tabsdiff/s", "frac": round(me_achieved / alu_peak, 4),
               "traffic": tr.get("me_sad_kernel") if world == 1 else None,
               "peak_source": f"148 SM x {VABSDIFF4_PER_CLK_SM} VABSDIFF4/clk (measured) x 4 x sm_max_mhz",
               "per_launch_ms": round(me_launch_ms, 4), "algorithmic_ops_per_launch": me_ops}
    dominant = roof_jac if jac_ms >= me_ms else roof_me

    # ---- the same pass kernel in its HBM-bound regime (north_star's >= 70 % HBM target):
    # J3's state with time tile 8 (8 / Tt = 1 B per update), one launch per pass, on a copy
    # of the state; not part of the step
    roof_hbm = None
    if world == 1:
        tt_h, passes_h = 8, 16
        b = a.clone()
        wb = torch.empty_like(b)
        sp.jacobi1d_timetiled(b, tt_h * passes_h, tt_h, 0, work=wb)
        torch.cuda.synchronize()
        e0.record(stream)
        for _ in range(2):
            sp.jacobi1d_timetiled(b, tt_h * passes_h, tt_h, 0, work=wb)
        e1.record(stream)
        torch.cuda.synchronize()
        pass_ms = e0.elapsed_time(e1) / (2 * passes_h)
        hb = 8.0 * n_local  # algorithmic bytes per pass: one read + one write of the state
        roof_hbm = {"kernel": "jacobi1d_pass_kernel", "config": f"J3 state, time tile {tt_h}, one launch per pass",
                    "bound": "hbm", "achieved": round(hb / (pass_ms * 1e-3) / 1e9, 1), "peak": pk["hbm_gbs"],
                    "unit": "GB/s", "frac": round(hb / (pass_ms * 1e-3) / 1e9 / pk["hbm_gbs"], 4),
                    "per_launch_ms": round(pass_ms, 4), "algorithmic_bytes_per_launch": hb,
                    "peak_source": pk["source"]}
        del b, wb

    # ---- end-to-end through the public API with host buffers (pinned H2D / D2H in the timed region)
    e2e = None
    me_e2e = None
    if world == 1:
        a_pin = torch.from_numpy(sp_inputs.jacobi_input(n_local, seed=sp_inputs.JACOBI_BENCH_SEED)).pin_memory()
        f_pin = torch.from_numpy(frames_host).pin_memory()
        # host-buffer Jacobi (sp_jacobi1d_host, wavefront order): a_pin moves in by copy-engine
        # chunks that release their pass-0 tiles, the last pass writes the result back over
        # PCIe itself; in place: every call advances the state T steps
        # (same time tile as the device-resident run unless --e2e-time-tile says otherwise)
        tt_e2e = args.e2e_time_tile or tt
        jac_host = sp.Jacobi1DHost(n_local, T, tt_e2e)
        # host-buffer ME: frames streamed frame by frame while the search runs, MV / SAD stored
        # into pinned host memory by the kernel (sp_me_search_host)
        me_host = sp.MESearchHost(ME_PAIRS + 1, ME_W, ME_H, frames_host.shape[2], ME_R)
        jac_host.run(a_pin)
        me_host.run(f_pin)
        torch.cuda.synchronize()
        ke = max(1, min(K, 3))
        tj = tm = 0.0
        for _ in range(ke):
            t0 = time.perf_counter()
            jac_host.run(a_pin)
            torch.cuda.synchronize()
            t1 = time.perf_counter()
            me_host.run(f_pin)
            torch.cuda.synchronize()
            t2 = time.perf_counter()
            tj += t1 - t0
            tm += t2 - t1
        # Jacobi's own bytes: the state read from and written back to pinned host memory
        e2e = {"value": (n_local - 2) * T * ke / tj / 1e9, "unit": "GPoint-updates/s",
               "h2d_bytes_per_step": 4 * n_local, "d2h_bytes_per_step": 4 * n_local,
               "api": "sp_jacobi1d_host (input: copy-engine chunks into device memory, each releasing its pass-0 tiles; output: the last pass TMA-stores into the pinned array; wavefront order)", "time_tile": tt_e2e}
        me_e2e = {"value": me_valid_sads(ME_W, ME_H, ME_R, ME_PAIRS) * ke / tm / 1e9, "unit": "GSAD/s",
                  "h2d_bytes_per_step": frames_host.nbytes, "d2h_bytes_per_step": ME_PAIRS * mby * mbx * 8,
                  "api": "sp_me_search_host (per-frame H2D overlapped with the search, outputs stored to pinned host)"}
    else:
        # every rank: its slab from pinned host memory -> the fused multi-GPU call -> back to
        # pinned host memory; wall clock per step, max over ranks
        slab_pin = torch.from_numpy(sp_inputs.jacobi_input(n_local, seed=sp_inputs.JACOBI_BENCH_SEED,
                                                           begin=x_begin)).pin_memory()
        ke = max(1, min(K, 2))
        walls = []
        for _ in range(ke + 1):  # (the first round is a warm-up)
            dist.barrier()
            t0 = time.perf_counter()
            a[H:H + n_local].copy_(slab_pin, non_blocking=True)
            jacobi_run(T)
            slab_pin.copy_(a[H:H + n_local], non_blocking=True)
            torch.cuda.synchronize()
            walls.append(time.perf_counter() - t0)
        tj = max_over_ranks(sum(walls[1:]))
        e2e = {"value": (n_global - 2) * T * ke / tj / 1e9, "unit": "GPoint-updates/s",
               "h2d_bytes_per_step": 4 * n_global, "d2h_bytes_per_step": 4 * n_global,
               "api": "pinned slab H2D + PeerSlab.run (sp_jacobi1d_timetiled_peer_fused) + D2H on every rank"
                      if slab is not None else "pinned slab H2D + Comm.jacobi1d_timetiled_dist + D2H on every rank"}

    # ---- CPU baseline: the oracle on a bounded sample (rank 0, N = 1 only)
    cpu = None
    if world == 1 and not args.no_cpu_baseline:
        cpu = cpu_baseline_obj(oracle_samples())

    # our kernels per step: Jacobi (1 persistent launch, or one per pass) (+ peer done signal)
    # + ME (1 launch; + the gather wait kernel)
    jac_l = (1 if persistent else -(-T // tt)) + (1 if slab is not None else 0)
    me_l = 1 + (1 if (me_shard is not None and args.gather == "peer") else 0)
    line = {
        "metric": METRIC, "value": round(jac_val, 2), "unit": "GPoint-updates/s", "n_gpus": world, "steps": K,
        "warmup": args.warmup, "ms_per_step": round(total_ms / K, 4), "higher_is_better": True,
        "scaling": "weak" if world == 1 else "strong",
        "vs_baseline": None, "dtype": "f32/u8", "data": "synthetic",
        "config": bench_config(world, tt, args.halo, args.gather),
        "jacobi": {"value": round(jac_val, 2), "unit": "GPoint-updates/s", "ms_per_step": round(jac_ms / K, 4),
                   "n_local": n_local, "passes_per_step": -(-T // tt),
                   # the persistent launches (single GPU and peer-fused) take the in-place
                   # geometry at Tt >= 48, the staged one below (include/sp.h sp_jacobi_plan)
                   "space_tile": sp.jacobi1d_plan(n_local, T, tt, 0)["persistent_space_tile" if persistent
                                                                      else "space_tile"],
                   "geometry": _geometry(n_local, T, tt, persistent)},
        "me": {"value": round(me_val, 2), "unit": "GSAD/s", "abs_diff_per_s": me_val * 256e9,
               "ms_per_step": round(me_ms / K, 4), "roofline": roof_me, "e2e": me_e2e},
        "roofline": dominant, "roofline_jacobi": roof_jac, "roofline_jacobi_hbm_regime": roof_hbm,
        "step_stats": step_stats,
        "cpu_baseline": cpu, "e2e": e2e, "gpu_launches": (jac_l + me_l) * K, "clocks": clk.summary(),
    }
    if rank == 0:
        print(json.dumps(line), flush=True)
    if comm is not None:
        comm.destroy()
    if slab is not None:
        slab.close()
    if me_shard is not None:
        me_shard.close()
    return 0


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def launch_cmd(argv, gpus, port=None):
    """The torchrun command bench.py runs itself under for --gpus N > 1 (one process per GPU
    of this node, rendezvous on 127.0.0.1)."""
    return [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={gpus}",
            "--master-addr=127.0.0.1", f"--master-port={port or _free_port()}", os.path.abspath(__file__), *argv]


def main(argv=None):
    argv = sys.argv[1:] if argv is None else argv
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    # Tt = 128: fastest on J3 with the persistent in-place geometry (K = 56: 6.41 ms vs 6.50 at
    # Tt = 64; profiles/r02_jacobi_inplace.txt r3p) — the time tile is the paper's own tuning
    # parameter (§4.3 tile-size search), not part of the J3 / J5 problem definitions
    ap.add_argument("--time-tile", type=int, default=128)
    ap.add_argument("--e2e-time-tile", type=int, default=0, help="time tile of the N = 1 host-buffer e2e call (0: --time-tile)")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--halo", choices=["peer", "nccl"], default="peer",
                    help="multi-GPU Jacobi halo exchange: fused peer stores in the pass kernel, or NCCL send/recv")
    ap.add_argument("--gather", choices=["peer", "nccl"], default="peer",
                    help="multi-GPU ME result all-gather: fused peer stores in the search kernel, or NCCL broadcasts")
    args = ap.parse_args(argv)
    if args.impl == "ours" and args.gpus > 1 and "WORLD_SIZE" not in os.environ:
        return subprocess.call(launch_cmd(argv, args.gpus))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local_rank = int(os.environ.get("LOCAL_RANK", "0"))
    if args.impl == "reference":
        return run_reference(args, rank, world)
    if world != args.gpus:
        raise SystemExit(f"--gpus {args.gpus} but WORLD_SIZE={world}: launch one process per GPU")
    # test hook: SP_BENCH_SHARE_GPU=1 runs every rank on cuda:0 with a gloo process group, to
    # exercise the multi-rank path on a one-GPU box (timings are then meaningless)
    share = os.environ.get("SP_BENCH_SHARE_GPU") == "1"
    if share:
        local_rank = 0
    if world > 1:
        import torch
        import torch.distributed as dist
        torch.cuda.set_device(local_rank)
        if share:
            dist.init_process_group("gloo")
        else:
            dist.init_process_group("nccl", device_id=torch.device("cuda", local_rank))
    try:
        return run_ours(args, rank, world, local_rank)
    finally:
        if world > 1:
            import torch.distributed as dist
            dist.destroy_process_group()


if __name__ == "__main__":
    sys.exit(main())
