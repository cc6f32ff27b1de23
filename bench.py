#!/usr/bin/env python
"""Benchmark of the perforated stencil hot path (BASELINE.json metric:
Mpixel/s and speedup vs the exact kernel at the stated mean relative error;
HBM GB/s).

Default workload (N=1): BASELINE configs[1] (C2) -- Gaussian 5x5 fp32 on
4096x4096 synthetic "natural" frames, row perforation, skipped fraction 1/2,
linear-interpolation reconstruction (the paper's Rows1:LI).  A step is one
perf_run over a batch of BATCH frames (512 MiB in + 512 MiB out, > L2, so no
flush is needed between steps).  The remaining C2 variants (Gaussian5 and
Sobel3 x row/col/checker x NN/LI x skipped 1/2, 1/4, 3/4) are timed the same
way after the headline and reported under "variants".

  python bench.py [--gpus N] [--steps K] [--warmup W] [--config C2|C1|C3|C4|C5] [--impl reference]

Under torchrun each rank runs its own batch (weak scaling, no data-path
collective); the timed region is bracketed by barriers + synchronize and the
max over ranks is reported.  --impl reference times the CPU oracle (the
paper-derived reference of this tier) on a bounded sample on rank 0.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "Mpixel/s (and speedup vs exact kernel) at stated mean relative error; HBM GB/s"

CONFIGS = {
    "C1": dict(app="gaussian", r=2, W=512, H=512, batch=512, scheme="row", rate=(1, 2), recon="li",
               cls="natural", seed=0x5EED0001, workload="C1: Gaussian 5x5 fp32 512x512, row 1/2, LI"),
    "C2": dict(app="gaussian", r=2, W=4096, H=4096, batch=8, scheme="row", rate=(1, 2), recon="li",
               cls="natural", seed=0x5EED0011,
               workload="C2: Gaussian 5x5 fp32 4096x4096, row perforation 1/2, LI (headline of the C2 sweep)"),
    "C3": dict(app="median", r=1, W=8192, H=8192, batch=4, scheme="col", rate=(1, 2), recon="nn",
               cls="natural", seed=0x5EED0020, workload="C3: Median 3x3 u8 8192x8192, column perforation 1/2, NN"),
    "C4": dict(app="hotspot", r=1, W=16384, H=16384, iters=200, scheme="row", rate=(1, 2), recon="li",
               seed=0x5EED0030, workload="C4: Hotspot fp32 16384x16384, 200 iterations, row perforation 1/2, LI"),
    "C5": dict(app="gauss_sobel", r=2, W=3840, H=2160, batch=16, scheme="row", rate=(1, 2), recon="li",
               cls="natural", seed=0x5EED1000,
               workload="C5: Gaussian5->Sobel3 fp32 3840x2160 frames, row perforation 1/2, LI"),
}


def kept_fraction(scheme, rate):
    num, den = rate
    return 1.0 if scheme == "none" or num == 0 else 1.0 - num / den


def bytes_per_px(app, scheme, rate):
    """algorithmic bytes per output pixel: kept input + full output (DESIGN.md Roofline)"""
    k = kept_fraction(scheme, rate)
    if app == "median":
        return k * 1 + 1
    if app == "hotspot":
        return k * 8 + 4  # T and P kept, T' written
    return k * 4 + 4


def load_peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        d = json.load(open(p))
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json copy)"
    return 6650.0, "fallback (B200_PROFILING.md)"


def ncu_entry(config, kernel_key):
    """per-launch ncu counters of this config's kernel in bench's launch
    configuration (profiles/ncu_traffic.json, written by tools/ncu_traffic.py)"""
    p = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    if not os.path.exists(p):
        return None
    try:
        return json.load(open(p)).get(f"{config}/{kernel_key}")
    except Exception:
        return None


def ncu_traffic(config, kernel_key):
    e = ncu_entry(config, kernel_key)
    return e["traffic"] if e else None


_bwp = None
_mix_cache = {}


def mixed_peak_gbs(in_ptr, out_ptr, out_bytes, scheme, rate, gran_bytes=128, n_in=1, stream=0, pitch_bytes=16384):
    """GB/s a plain streaming kernel reaches with the same read/write mix and the
    same per-CTA footprint as a perforated stencil (tools/bwprobe.cu, measured on
    this box): every output byte written once, the kept fraction of the input read
    (whole rows for the row scheme / exact, gran_bytes cells for column /
    checker), each CTA streaming 4-KB x 128-row blocks, best of 4 / 8 CTAs per SM.
    Algorithmic bytes over the probe's time: comparable to roofline.achieved."""
    global _bwp
    import ctypes
    if _bwp is None:
        _bwp = ctypes.CDLL(os.path.join(ROOT, "tools", "libbwprobe.so"))
        _bwp.bwp_time_ms.restype = ctypes.c_float
        _bwp.bwp_time_ms.argtypes = [ctypes.c_void_p, ctypes.c_void_p, ctypes.c_longlong, ctypes.c_int,
                                     ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_void_p]
        _bwp.bwp_block_ms.restype = ctypes.c_float
        _bwp.bwp_block_ms.argtypes = [ctypes.c_void_p, ctypes.c_void_p, ctypes.c_longlong, ctypes.c_longlong,
                                      ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int,
                                      ctypes.c_int, ctypes.c_int, ctypes.c_void_p]
    num, den = rate
    if scheme == "none" or num == 0:
        kn, kd = 1, 1
    else:
        kd = den
        kn = den - num
    unit = pitch_bytes if scheme in ("none", "row") else gran_bytes
    key = (out_bytes, kn, kd, unit, n_in, pitch_bytes)
    if key not in _mix_cache:
        ms = _bwp.bwp_block_ms(in_ptr, out_ptr, out_bytes, pitch_bytes, 4096, 128, kn, kd, unit, n_in, 3, stream)
        k = kn / kd
        _mix_cache[key] = (n_in * k + 1.0) * out_bytes / (ms * 1e-3) / 1e9 if ms > 0 else None
    return _mix_cache[key]


class ClockSampler:
    FIELDS = ("clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.hw_slowdown,"
              "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
              "clocks_event_reasons.sw_power_cap")

    def __init__(self, index):
        self.index = index
        self.rows = []
        self.proc = None

    def __enter__(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.index), f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                 "-lms", "100"], stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
            time.sleep(0.3)
        except Exception:
            self.proc = None
        return self

    def _read(self):
        for line in self.proc.stdout:
            parts = [x.strip() for x in line.split(",")]
            if len(parts) >= 7:
                self.rows.append(parts)

    def __exit__(self, *a):
        if self.proc:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=2)
            except Exception:
                self.proc.kill()

    def summary(self):
        if not self.rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unsampled"]}
        sm = [float(r[0]) for r in self.rows if r[0].replace(".", "").isdigit()]
        mx = [float(r[1]) for r in self.rows if r[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in self.rows for i in range(4) if r[3 + i].lower() == "active"})
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": reasons, "samples": len(self.rows)}


def dist_setup(args):
    import torch
    ws = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    # KPERF_BENCH_BACKEND=gloo lets several ranks share one GPU (code-path test on a
    # 1-GPU box; NCCL refuses two ranks on one device).  Production: nccl, one GPU per rank.
    backend = os.environ.get("KPERF_BENCH_BACKEND", "nccl")
    dev = local % max(1, torch.cuda.device_count())
    if ws > 1:
        import torch.distributed as dist
        os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
        torch.cuda.set_device(dev)
        if backend == "nccl":
            dist.init_process_group("nccl", device_id=torch.device("cuda", dev))
        else:
            dist.init_process_group(backend)
    else:
        torch.cuda.set_device(0)
    return ws, rank, dev


def barrier(ws):
    if ws > 1:
        import torch.distributed as dist
        dist.barrier()


def max_over_ranks(ws, v):
    if ws == 1:
        return v
    import torch
    import torch.distributed as dist
    on_gpu = dist.get_backend() == "nccl"
    t = torch.tensor([v], dtype=torch.float64, device="cuda" if on_gpu else "cpu")
    dist.all_reduce(t, op=dist.ReduceOp.MAX)
    return float(t.item())


def nccl_uid(kp, ws, rank):
    """a libkperf NCCL unique id from rank 0, broadcast over the process group"""
    import torch
    import torch.distributed as dist
    uid = kp.perf_comm_unique_id() if rank == 0 else bytes(128)
    t = torch.tensor(list(uid), dtype=torch.uint8, device="cuda" if dist.get_backend() == "nccl" else "cpu")
    dist.broadcast(t, 0)
    return bytes(t.cpu().tolist())


def min_over_ranks(ws, v):
    return -max_over_ranks(ws, -v)


def time_kernel(fn, stream, reps, warm):
    """average device time per call (ms), CUDA events on the launching stream"""
    import torch
    for _ in range(warm):
        fn()
    torch.cuda.synchronize()
    a = torch.cuda.Event(enable_timing=True)
    b = torch.cuda.Event(enable_timing=True)
    a.record(stream)
    for _ in range(reps):
        fn()
    b.record(stream)
    b.synchronize()
    return a.elapsed_time(b) / reps


# ---------------------------------------------------------------------------
def oracle_sample(cfg, rows=256):
    """time the oracle (as it stands, single-threaded) on a bounded sample:
    the first `rows` rows of one frame of the config (fresh image each call)."""
    import oracle
    import synth
    app, W = cfg["app"], cfg["W"]
    if app == "hotspot":
        n = min(cfg["W"], 1024)
        T, P = _sample_input(cfg, n, rows)
        prm = oracle.params("hotspot", n, rows, 1, cfg["scheme"], cfg["rate"], cfg["recon"])
        t0 = time.perf_counter()
        oracle.hotspot(prm, T, P, 1)
        return (n * rows) / (time.perf_counter() - t0), f"1 Hotspot step on a {n}x{rows} grid"
    u8 = app == "median"
    img = _sample_input(cfg, W, rows)
    prm = oracle.params(app, W, rows, cfg["r"], cfg["scheme"], cfg["rate"], cfg["recon"], 128 if u8 else 32)
    t0 = time.perf_counter()
    oracle.run(prm, img)
    return (W * rows) / (time.perf_counter() - t0), f"{W}x{rows} rows of one frame"


def host_cores():
    try:
        return len(os.sched_getaffinity(0))
    except Exception:
        return os.cpu_count() or 1


def cpu_model():
    try:
        for line in open("/proc/cpuinfo"):
            if line.startswith("model name"):
                return line.split(":", 1)[1].strip()
    except Exception:
        pass
    return "unknown"


_samples = {}


def _sample_input(cfg, W, rows):
    """the synthetic sample the CPU legs run on (generated once per shape)"""
    import synth
    key = (cfg["workload"], W, rows)
    if key not in _samples:
        if cfg["app"] == "hotspot":
            _samples[key] = synth.hotspot(cfg["seed"], W, rows)
        else:
            _samples[key] = synth.image(cfg["cls"], cfg["seed"], W, rows,
                                        np.uint8 if cfg["app"] == "median" else np.float32)
    return _samples[key]


def oracle_sample_bands(cfg, rows=256, threads=None, check=False):
    """the same oracle, band-parallel over the host cores: the
    sample's rows are cut into `threads` bands; each band runs oracle.run /
    oracle.hotspot on its rows plus a halo in its own thread (the C oracle runs
    without the GIL), and the band's own rows are kept.  Band starts are
    aligned to the perforation period and the halo covers radius + rebuild
    distance, so the stitched result equals the single-threaded run (check)."""
    import concurrent.futures as cf

    import oracle
    import synth
    threads = threads or host_cores()
    app, W = cfg["app"], cfg["W"]
    den = cfg["rate"][1]
    align = int(np.lcm(den, 16))
    r = 1 if app == "hotspot" else (3 if app == "gauss_sobel" else cfg["r"])
    halo = -(-(r + den) // align) * align
    per = -(-(-(-rows // threads)) // align) * align
    cuts = list(range(0, rows, per)) + [rows]
    if app == "hotspot":
        n = min(W, 1024)
        T, P = _sample_input(cfg, n, rows)
        whole = lambda: oracle.hotspot(oracle.params("hotspot", n, rows, 1, cfg["scheme"], cfg["rate"],  # noqa: E731
                                                     cfg["recon"]), T, P, 1)

        def band(k):
            a, b = max(0, cuts[k] - halo), min(rows, cuts[k + 1] + halo)
            o = oracle.hotspot(oracle.params("hotspot", n, b - a, 1, cfg["scheme"], cfg["rate"], cfg["recon"]),
                               np.ascontiguousarray(T[a:b]), np.ascontiguousarray(P[a:b]), 1)
            return o[cuts[k] - a:cuts[k + 1] - a]
        px, desc = n * rows, f"1 Hotspot step on a {n}x{rows} grid"
    else:
        u8 = app == "median"
        img = _sample_input(cfg, W, rows)
        G = 128 if u8 else 32
        whole = lambda: oracle.run(oracle.params(app, W, rows, cfg["r"], cfg["scheme"], cfg["rate"],  # noqa: E731
                                                 cfg["recon"], G), img)

        def band(k):
            a, b = max(0, cuts[k] - halo), min(rows, cuts[k + 1] + halo)
            o = oracle.run(oracle.params(app, W, b - a, cfg["r"], cfg["scheme"], cfg["rate"], cfg["recon"], G),
                           np.ascontiguousarray(img[a:b]))
            return o[cuts[k] - a:cuts[k + 1] - a]
        px, desc = W * rows, f"{W}x{rows} rows of one frame"
    with cf.ThreadPoolExecutor(max_workers=threads) as ex:
        t0 = time.perf_counter()
        parts = list(ex.map(band, range(len(cuts) - 1)))
        dt = time.perf_counter() - t0
    same = None
    if check:
        # rows within halo of the sample's own top / bottom see the sample's border (both runs alike)
        same = bool(np.array_equal(np.concatenate(parts), whole()))
    return px / dt, desc, len(cuts) - 1, same


def cpu_baseline(cfg, budget_s=10.0):
    """the oracle as it stands on the box's host cores: single-threaded (the
    headline CPU figure) and band-parallel over every core (same code, same
    results), each on a bounded sample of about budget_s seconds"""
    px = 0.0
    t = 0.0
    n = 0
    desc = ""
    while t < budget_s and n < 200:
        rate, desc = oracle_sample(cfg)
        # rate = px/s for this call; accumulate time-weighted
        px_call = cfg["W"] * 256 if cfg["app"] != "hotspot" else min(cfg["W"], 1024) * 256
        px += px_call
        t += px_call / rate
        n += 1
    unit = "Mpixel/s" if cfg["app"] != "hotspot" else "Mcell-updates/s"
    cores = host_cores()
    rows_mt = min(4096, max(1024, 128 * cores))  # >= 32-row bands, one per core
    threads = max(1, min(cores, rows_mt // 32))
    pxm, tm, nm, same = 0.0, 0.0, 0, None
    while tm < budget_s / 2 and nm < 50:
        rate, desc_mt, bands, ok = oracle_sample_bands(cfg, rows_mt, threads, check=(nm == 0))
        if nm == 0:
            same = ok
        px_call = (cfg["W"] if cfg["app"] != "hotspot" else min(cfg["W"], 1024)) * rows_mt
        pxm += px_call
        tm += px_call / rate
        nm += 1
    return {"value": px / t / 1e6, "unit": unit, "cores": 1, "kind": "oracle",
            "sample": f"{n} x oracle.run on {desc} ({t:.1f} s of CPU work)",
            "cpu_model": cpu_model(), "nproc": cores,
            "all_cores": {"value": pxm / tm / 1e6, "unit": unit, "cores": cores, "kind": "oracle, band-parallel",
                          "sample": f"{nm} x {bands} bands of {desc_mt} on {threads} threads ({tm:.1f} s wall)",
                          "identical_to_single_thread": same}}


def run_reference(args, ws, rank):
    cfg = CONFIGS[args.config]
    if rank != 0:
        return
    unit = "Mpixel/s" if cfg["app"] != "hotspot" else "Mcell-updates/s"
    for _ in range(args.warmup):
        oracle_sample(cfg)
    rates, t_total, px_total = [], 0.0, 0
    for _ in range(args.steps):
        r, desc = oracle_sample(cfg)
        px = cfg["W"] * 256 if cfg["app"] != "hotspot" else min(cfg["W"], 1024) * 256
        t_total += px / r
        px_total += px
    v = px_total / t_total / 1e6
    line = {"impl": "reference", "metric": METRIC, "value": v, "unit": unit, "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": 1e3 * t_total / args.steps,
            "higher_is_better": True, "scaling": "weak", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
            "config": {"workload": cfg["workload"], "sample": f"each step: oracle.run on {desc}"},
            "cpu_baseline": {"value": v, "unit": unit, "cores": 1, "kind": "oracle",
                             "sample": f"{args.steps} steps of oracle.run on {desc}", "cpu_model": cpu_model(),
                             "nproc": host_cores()},
            "e2e": {"value": v, "unit": unit, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


# ---------------------------------------------------------------------------
def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=5)
    ap.add_argument("--config", default="C2", choices=sorted(CONFIGS))
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--no-variants", action="store_true")
    ap.add_argument("--sweep", action="store_true",
                    help="print only the C2 sweep (3 input classes x variants, incl. G = 1 px cells) as one JSON line")
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--batch", type=int, default=0)
    ap.add_argument("--halo", default="nccl", choices=["nccl", "p2p"],
                    help="C4 with N > 1: halo exchange by NCCL send/recv or (NEXT-4) peer stores fused "
                         "into the step kernels over NVLink (CUDA IPC + epoch flags)")
    ap.add_argument("--tblock", type=int, default=1,
                    help="C4 only: Hotspot steps per launch (temporal blocking, DESIGN.md R19); 1 = per-step")
    args = ap.parse_args()
    args.warmup = max(args.warmup, 3)

    if args.impl == "reference":
        ws = int(os.environ.get("WORLD_SIZE", "1"))
        rank = int(os.environ.get("RANK", "0"))
        run_reference(args, ws, rank)
        return

    import torch

    import paper_conf_cgo_maiercj18_b200 as kp
    import synth

    ws, rank, local = dist_setup(args)
    cfg = dict(CONFIGS[args.config])
    if args.batch:
        cfg["batch"] = args.batch
    stream = torch.cuda.current_stream()
    peak, peak_src = load_peaks()
    app, W, H = cfg["app"], cfg["W"], cfg["H"]
    u8 = app == "median"
    es = 1 if u8 else 4
    unit = "Mpixel/s" if app != "hotspot" else "Mcell-updates/s"

    if args.sweep:
        if rank == 0:
            print(json.dumps(bench_sweep(kp, stream, peak)), flush=True)
        return
    if app == "hotspot":
        result = bench_hotspot(args, cfg, ws, rank, local, stream, peak, peak_src)
    else:
        B = cfg["batch"]
        dt = torch.uint8 if u8 else torch.float32
        x = torch.empty((B, H, W), dtype=dt, device="cuda")
        # per-rank distinct frames: seed + rank * B + f
        synth.image_device(cfg["cls"], cfg["seed"] + rank * B, W, H, B, x.data_ptr(), u8, stream.cuda_stream)
        y = torch.empty_like(x)
        yex = torch.empty_like(x)
        G = 128  # the measured B200 DRAM fill granule (tools/granule_probe.cu)
        plan = kp.Plan(app, W, H, cfg["r"], cfg["scheme"], cfg["rate"], cfg["recon"], batch=B, granule_bytes=G)
        exact = kp.Plan(app, W, H, cfg["r"], "none", (0, 1), "nn", batch=B)
        run = lambda: plan.run(x, y, stream)  # noqa: E731
        # (the warm-up runs inside the clock sampler: its start-up pause would
        # otherwise leave the GPU idle for 0.3 s right before the timed steps)
        with ClockSampler(local) as clk:
            for _ in range(args.warmup):
                run()
            torch.cuda.synchronize()
            barrier(ws)
            torch.cuda.synchronize()
            e0 = torch.cuda.Event(enable_timing=True)
            e1 = torch.cuda.Event(enable_timing=True)
            e0.record(stream)
            for _ in range(args.steps):
                run()
            e1.record(stream)
            e1.synchronize()
        torch.cuda.synchronize()
        barrier(ws)
        ms = max_over_ranks(ws, e0.elapsed_time(e1) / args.steps)
        px_step = B * W * H
        value = ws * px_step / (ms * 1e-3) / 1e6
        # exact kernel, same batch (speedup) and error at the stated MRE
        ms_exact = max_over_ranks(ws, time_kernel(lambda: exact.run(x, yex, stream), stream, args.steps,
                                                  args.warmup))
        if ws > 1:  # the error of the whole sharded batch: partial sums ncclAllReduce'd
            uid = nccl_uid(kp, ws, rank)
            try:
                kp.perf_comm_init(plan.handle, uid, rank, ws)
                mre, cnt = kp.perf_error_allreduce(plan.handle, yex, y, stream)
            except kp.PerfError:  # (KPERF_BENCH_BACKEND=gloo test mode: ranks share a GPU, NCCL refuses)
                import torch.distributed as dist
                sums = torch.tensor(kp.perf_error_sums(plan.handle, yex, y, stream), dtype=torch.float64)
                dist.all_reduce(sums)
                mre, cnt = kp.perf_error_finish(plan.handle, sums.tolist())
        else:
            mre, cnt = plan.error(yex, y, stream)
        # a5, the error kernel (two deterministic passes + an 24-B read-back), timed alone
        err_ms = []
        for _ in range(4):
            ea, eb = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            ea.record(stream)
            kp.perf_error_sums(plan.handle, yex, y, stream)
            eb.record(stream)
            eb.synchronize()
            err_ms.append(ea.elapsed_time(eb))
        err_ms = sorted(err_ms)[len(err_ms) // 2]
        err_kernel = {"ms": err_ms, "bytes": 2 * px_step * es, "gbs": 2 * px_step * es / (err_ms * 1e-3) / 1e9,
                      "note": "perf_error_sums: partial pass (592 x 256 threads, 16-B loads) + one-block tree, "
                              "read-back of 3 fp64 included"}
        algo_b = bytes_per_px(app, cfg["scheme"], cfg["rate"]) * px_step
        achieved = algo_b / (ms * 1e-3) / 1e9
        kkey = f"{app}{cfg['r']}_{cfg['scheme']}_{cfg['rate'][0]}-{cfg['rate'][1]}_{cfg['recon']}"
        tr = ncu_traffic(args.config, kkey)
        clk_sum = clk.summary()
        alu = None
        ent = ncu_entry(args.config, kkey)
        if u8 and ent:  # the median is ALU-pipe bound: a pipe-resolved roofline
            # achieved = ALU-pipe warp instructions of this launch (ncu, same launch configuration)
            # / the launch's CUDA-event time; peak = the ALU pipe's issue rate, 0.5 warp-instruction
            # per cycle per SM sub-partition (16 lanes/clk), x 4 x 148 at the SM clock sampled here
            sm_mhz = clk_sum.get("sm_mhz") or 1965.0
            alu_peak = 0.5 * 4 * 148 * sm_mhz * 1e6 / 1e9  # G warp-inst/s
            alu_ach = ent["warp_inst_pipe_alu"] / (ms * 1e-3) / 1e9
            alu = {"bound": "alu", "achieved": alu_ach, "peak": alu_peak, "unit": "Gwarp-inst/s (ALU pipe)",
                   "frac": alu_ach / alu_peak, "traffic": tr, "kernel": kkey,
                   "warp_inst_pipe_alu_per_launch": ent["warp_inst_pipe_alu"],
                   "warp_inst_pipe_fma_per_launch": ent["warp_inst_pipe_fma"],
                   "ncu_pipe_alu_pct_of_peak": ent["pipe_alu_pct_of_peak"],
                   "peak_derivation": f"148 SM x 4 SMSP x 0.5 ALU warp-inst/clk x {sm_mhz:.0f} MHz (sampled)",
                   "source": "profiles/ncu_traffic.json (tools/ncu_traffic.py)"}
        pmix = mixed_peak_gbs(x.data_ptr(), yex.data_ptr(), px_step * es, cfg["scheme"], cfg["rate"], G,
                              stream=stream.cuda_stream, pitch_bytes=W * es) if not u8 else None
        result = {
            "metric": METRIC, "value": value, "unit": unit, "n_gpus": ws, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True, "scaling": "weak",
            "vs_baseline": None, "dtype": "u8" if u8 else "f32", "data": "synthetic",
            "config": {"workload": cfg["workload"], "W": W, "H": H, "frames_per_gpu": B,
                       "granule_bytes": G, "l2": "inputs larger than L2 (batch of frames, no flush)",
                       "parallelism": f"frames sharded, {B} per GPU" if ws > 1 else "single GPU"},
            "speedup_vs_exact": ms_exact / ms, "exact_ms_per_step": ms_exact,
            "exact_mpixel_s": ws * px_step / (ms_exact * 1e-3) / 1e6,
            "error": {"metric": "mre" if app not in ("sobel", "gauss_sobel") else "me", "value": mre,
                      "count": cnt, "over": f"all {ws} ranks' frames (perf_error_allreduce)" if ws > 1
                      else "the batch"},
            "hbm_gbs": achieved,
            "error_kernel": err_kernel,
            "roofline": {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s",
                         "frac": achieved / peak, "traffic": tr, "kernel": kkey,
                         "algorithmic_bytes_per_launch": algo_b, "peak_source": peak_src,
                         "peak_mix": pmix, "frac_mix": achieved / pmix if pmix else None,
                         "peak_mix_source": "tools/bwprobe.cu on this box: plain stream, same read/write mix and CTA footprint"},
            "clocks": clk_sum,
            "gpu_launches": args.steps,
        }
        if alu:
            result["roofline_hbm"] = result["roofline"]
            result["roofline"] = alu
        # e2e through the C ABI with pinned host buffers (one frame per step)
        result["e2e"] = bench_e2e(kp, cfg, stream, args, ws, x)
        if not args.no_variants and args.config == "C2":
            result["variants"] = bench_variants(kp, cfg, x, y, yex, stream, peak, ws)
        plan.close()
        exact.close()
        if ws > 1 and args.config == "C2":  # the paths that really exchange data between GPUs
            del x, y, yex
            torch.cuda.empty_cache()
            # watchdog: the headline line above is complete; if a row-band leg stalls (an NCCL
            # transport problem on some box), print it with the legs marked and leave
            def _timeout():
                for key in ("c4_row_bands", "c2_row_bands"):
                    result.setdefault(key, {"error": "timeout (watchdog, 300 s)"})
                if rank == 0:
                    print(json.dumps(result), flush=True)
                os._exit(0)
            wd = threading.Timer(float(os.environ.get("KPERF_BENCH_LEG_TIMEOUT", "300")), _timeout)
            wd.daemon = True
            wd.start()
            for key, fn in (("c4_row_bands", lambda: bench_c4_banded(kp, ws, rank, stream)),
                            ("c2_row_bands", lambda: bench_c2_row_bands(kp, ws, rank, stream, args.steps))):
                try:
                    result[key] = fn()
                except Exception as e:  # (e.g. NCCL refusing two ranks on one GPU under the gloo test mode)
                    result[key] = {"error": f"{type(e).__name__}: {e}"}
            wd.cancel()
    if rank == 0 and not args.no_cpu:
        result["cpu_baseline"] = cpu_baseline(cfg)
    if rank == 0:
        print(json.dumps(result), flush=True)
    if ws > 1:
        import torch.distributed as dist
        dist.destroy_process_group()


def bench_e2e(kp, cfg, stream, args, ws, x):
    import torch
    app, W, H = cfg["app"], cfg["W"], cfg["H"]
    u8 = app == "median"
    hin = x[0].cpu().pin_memory()
    hout = torch.empty_like(hin).pin_memory()
    plan = kp.Plan(app, W, H, cfg["r"], cfg["scheme"], cfg["rate"], cfg["recon"], batch=1)
    f = lambda: plan.run_host(hin, hout, stream)  # noqa: E731
    for _ in range(3):
        f()
    torch.cuda.synchronize()
    barrier(ws)
    steps = max(3, min(args.steps, 10))
    e0 = torch.cuda.Event(enable_timing=True)
    e1 = torch.cuda.Event(enable_timing=True)
    e0.record(stream)
    for _ in range(steps):
        f()
    e1.record(stream)
    e1.synchronize()
    ms = max_over_ranks(ws, e0.elapsed_time(e1) / steps)
    nb = W * H * (1 if u8 else 4)
    h2d = plan.get("h2d_bytes")  # row scheme: only the kept rows cross PCIe (PERF_KEY_HOST_SKIP)
    plan.close()
    return {"value": ws * W * H / (ms * 1e-3) / 1e6, "unit": "Mpixel/s" if app != "hotspot" else "Mcell-updates/s",
            "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": nb, "ms_per_step": ms,
            "api": "perf_run_host (pinned host buffers, one frame per step; row scheme: kept rows only host->device)"}


def bench_variants(kp, cfg, x, y, yex, stream, peak, ws):
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    px = B * W * H
    out = []
    for app, r in (("gaussian", 2), ("sobel", 1)):
        ex = kp.Plan(app, W, H, r, "none", (0, 1), "nn", batch=B)
        ms_ex = time_kernel(lambda: ex.run(x, yex, stream), stream, 10, 3)
        pm_ex = mixed_peak_gbs(x.data_ptr(), y.data_ptr(), px * 4, "none", (0, 1), 128, stream=stream.cuda_stream)
        out.append({"app": app, "r": r, "scheme": "none", "rate": [0, 1], "recon": "-", "ms": ms_ex,
                    "mpixel_s": px / ms_ex / 1e3, "speedup": 1.0, "error": 0.0,
                    "hbm_gbs": 8 * px / ms_ex / 1e6, "frac": 8 * px / ms_ex / 1e6 / peak,
                    "frac_mix": 8 * px / ms_ex / 1e6 / pm_ex if pm_ex else None})
        for scheme in ("row", "col", "checker"):
            for rate in ((1, 2), (1, 4), (3, 4)):
                for recon in ("nn", "li"):
                    p = kp.Plan(app, W, H, r, scheme, rate, recon, batch=B)
                    ms = time_kernel(lambda: p.run(x, y, stream), stream, 10, 3)
                    err, _ = p.error(yex, y, stream)
                    gbs = bytes_per_px(app, scheme, rate) * px / ms / 1e6
                    pm = mixed_peak_gbs(x.data_ptr(), y.data_ptr(), px * 4, scheme, rate, 128,
                                        stream=stream.cuda_stream)
                    pm_ex = mixed_peak_gbs(x.data_ptr(), y.data_ptr(), px * 4, "none", (0, 1), 128,
                                           stream=stream.cuda_stream)
                    out.append({"app": app, "r": r, "scheme": scheme, "rate": list(rate), "recon": recon,
                                "ms": ms, "mpixel_s": px / ms / 1e3, "speedup": ms_ex / ms, "error": err,
                                "hbm_gbs": gbs, "frac": gbs / peak, "frac_mix": gbs / pm if pm else None,
                                "byte_ceiling": 8.0 / bytes_per_px(app, scheme, rate),
                                "mix_ceiling": (pm / bytes_per_px(app, scheme, rate)) / (pm_ex / 8.0)
                                if pm and pm_ex else None})
                    p.close()
        for tile in ((16, 16), (32, 8)):  # NEXT-1: the paper's Stencil1 (halo-only perforation)
            p = kp.Plan(app, W, H, r, "stencil1", (0, 1), "nn", batch=B, tile1_w=tile[0], tile1_h=tile[1])
            ms = time_kernel(lambda: p.run(x, y, stream), stream, 10, 3)
            err, _ = p.error(yex, y, stream)
            out.append({"app": app, "r": r, "scheme": "stencil1", "tile": list(tile), "rate": [0, 1], "recon": "nn",
                        "ms": ms, "mpixel_s": px / ms / 1e3, "speedup": ms_ex / ms, "error": err,
                        "hbm_gbs": 8 * px / ms / 1e6, "frac": 8 * px / ms / 1e6 / peak,
                        "frac_mix": 8 * px / ms / 1e6 / pm_ex if pm_ex else None})
            p.close()
        ex.close()
    return out


def hotspot_cone_ok(cfg, W, Hg, iters, x0, y0, w, h, got, scheme, rate, recon):
    """oracle check of a w x h patch of a banded Hotspot result: the patch's
    dependency cone (iters x (1 + den) rows / iters columns each side) is
    generated on the device (synth, global rows), copied back and stepped by
    oracle.hotspot_window; rows / columns at the window's edge are wrong only
    outside the cone"""
    import torch

    import oracle
    import synth
    den = rate[1] if scheme in ("row", "checker") and rate[0] > 0 else 0
    my, mx = iters * (1 + den), iters
    wy0, wy1 = max(0, y0 - my), min(Hg, y0 + h + my)
    wx0, wx1 = max(0, x0 - mx), min(W, x0 + w + mx)
    T = torch.empty((wy1 - wy0, W), device="cuda")
    P = torch.empty_like(T)
    synth.hotspot_band_device(cfg["seed"], W, Hg, wy0, wy1 - wy0, T.data_ptr(), P.data_ptr())
    torch.cuda.synchronize()
    Tw = np.ascontiguousarray(T.cpu().numpy()[:, wx0:wx1].astype(np.float64))
    Pw = np.ascontiguousarray(P.cpu().numpy()[:, wx0:wx1])
    prm = oracle.params("hotspot", W, Hg, 1, scheme, rate, recon)
    oracle.hotspot_window(prm, Tw, Pw, wx0, wy0, iters)
    want = Tw[y0 - wy0:y0 - wy0 + h, x0 - wx0:x0 - wx0 + w]
    return bool(np.all(np.abs(got.astype(np.float64) - want) <= 1e-5 * np.abs(want)))


def bench_c4_banded(kp, ws, rank, stream, rows_per_gpu=2048, iters=20, reps=5):
    """the C4 Hotspot as row bands over the N ranks, per-launch
    NCCL halo exchange overlapped with the interior rows, the loop captured in
    a CUDA graph.  16384 x (rows_per_gpu x N) cells, `iters` steps per call
    (weak scaling).  Also timed with the exchange switched off
    (PERF_KEY_EXCHANGE 0, results wrong at band edges) to give the halo's
    share; each rank checks patches at both band edges against the oracle."""
    import torch

    import synth
    cfg = CONFIGS["C4"]
    W, Hg = cfg["W"], rows_per_gpu * ws
    scheme, rate, recon = cfg["scheme"], cfg["rate"], cfg["recon"]
    cuts = kp.band_cuts(Hg, ws)
    y0, h = cuts[rank], cuts[rank + 1] - cuts[rank]
    T = torch.empty((h, W), device="cuda")
    P = torch.empty_like(T)
    synth.hotspot_band_device(cfg["seed"], W, Hg, y0, h, T.data_ptr(), P.data_ptr(), stream.cuda_stream)
    out = torch.empty_like(T)
    uid = nccl_uid(kp, ws, rank)
    res = {"grid": [W, Hg], "iters_per_call": iters, "bands": ws, "scheme": scheme, "rate": list(rate),
           "recon": recon, "halo": "NCCL send/recv per launch, boundary rows first, exchange overlapped with the "
                                   "interior rows, loop captured in a CUDA graph"}
    times = {}
    for xchg in (1, 0):
        with kp.Plan("hotspot", W, h, 1, scheme, rate, recon, iters=iters, global_h=Hg, band_y0=y0,
                     exchange=xchg) as p:
            kp.perf_comm_init(p.handle, uid, rank, ws)
            run = lambda: p.hotspot(T, P, out, stream)  # noqa: E731
            barrier(ws)
            times[xchg] = max_over_ranks(ws, time_kernel(run, stream, reps, 2))
            if xchg:
                res["graph"] = p.get("graph")
                run()
                torch.cuda.synchronize()
                o = out.cpu().numpy()
                ok = True
                for x0, yy in ((1000, y0), (W - 4, y0 + h - 3), (8190, y0 + h // 2)):
                    ok &= hotspot_cone_ok(cfg, W, Hg, iters, x0, yy, 4, 3, o[yy - y0:yy - y0 + 3, x0:x0 + 4],
                                          scheme, rate, recon)
                res["parity"] = "ok" if min_over_ranks(ws, 1.0 if ok else 0.0) > 0 else "MISMATCH"
    cells = W * Hg * iters
    res.update({"ms_per_call": times[1], "mcell_updates_s": cells / (times[1] * 1e-3) / 1e6,
                "ms_per_call_no_exchange": times[0],
                "halo_us_per_step": max(0.0, times[1] - times[0]) * 1e3 / iters,
                "parity_check": "each rank: 4x3 patches at both band edges + the middle vs oracle.hotspot_window "
                                "on the dependency cone"})
    return res


def bench_c2_row_bands(kp, ws, rank, stream, steps):
    """one C2 batch (8 x 4096^2 fp32, Gaussian5 row 1/2 LI) split
    into N row bands; every step perf_run_band fills the halo rows of all
    frames with one NCCL group, then runs the band (strong scaling)"""
    import torch

    import synth
    cfg = CONFIGS["C2"]
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    cuts = kp.band_cuts(H, ws)
    y0, h = cuts[rank], cuts[rank + 1] - cuts[rank]
    uid = nccl_uid(kp, ws, rank)
    with kp.Plan(cfg["app"], W, h, cfg["r"], cfg["scheme"], cfg["rate"], cfg["recon"], batch=B, global_h=H,
                 band_y0=y0, granule_bytes=128) as p:
        kp.perf_comm_init(p.handle, uid, rank, ws)
        hp = kp.perf_band_halo(p.handle, rank, ws)
        hb = hp["halo_rows"]
        whole = torch.empty((B, H, W), device="cuda")
        synth.image_device(cfg["cls"], cfg["seed"], W, H, B, whole.data_ptr(), False, stream.cuda_stream)
        buf = torch.full((B, hp["buf_rows"], W), float("nan"), device="cuda")
        buf[:, hb:hb + h] = whole[:, y0:y0 + h]  # own rows only; halos arrive by NCCL
        del whole
        out = torch.empty((B, h, W), device="cuda")
        run = lambda: kp.perf_run_band(p.handle, buf, out, stream)  # noqa: E731
        barrier(ws)
        ms = max_over_ranks(ws, time_kernel(run, stream, steps, 3))
        # sampled parity: rows at both band edges of frame 1 vs the oracle
        import oracle
        img = synth.image(cfg["cls"], cfg["seed"] + 1, W, H)
        prm = oracle.params(cfg["app"], W, H, cfg["r"], cfg["scheme"], cfg["rate"], cfg["recon"])
        ys = np.r_[y0, y0 + 1, y0 + h - 2, y0 + h - 1]
        yy, xx = np.meshgrid(ys, np.arange(0, W, 11), indexing="ij")
        want = oracle.run_pixels(prm, img, xx.ravel(), yy.ravel())
        got = out[1].cpu().numpy()[yy.ravel() - y0, xx.ravel()]
        ok = bool(np.all(np.abs(got - want) <= 1e-5 * np.abs(want)))
    return {"workload": cfg["workload"] + f", one batch split into {ws} row bands", "ms_per_step": ms,
            "mpixel_s": B * W * H / (ms * 1e-3) / 1e6, "scaling": "strong", "halo_rows": hb,
            "parity": "ok" if min_over_ranks(ws, 1.0 if ok else 0.0) > 0 else "MISMATCH"}


def bench_sweep(kp, stream, peak, steps=10):
    """SURVEY 8(d) C2 sweep: the three synthetic input classes of Fig. 7
    (flat / natural / pattern) x {Gaussian5, Sobel3} x every
    row / column / checkerboard variant at 128-B cells, plus the pixel-granular
    (G = 1) column and checkerboard variants the paper's ">= 32 B" rule
     advises against.  Speedup vs the exact kernel on the same
    frames, error vs the exact output (MRE; Sobel: ME)."""
    import torch

    import synth
    cfg = CONFIGS["C2"]
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    px = B * W * H
    x = torch.empty((B, H, W), device="cuda")
    y, yex = torch.empty_like(x), torch.empty_like(x)
    out = []
    for cls in ("flat", "natural", "pattern"):
        synth.image_device(cls, synth.SEED_C2 + synth.CLASSES[cls], W, H, B, x.data_ptr(), False, stream.cuda_stream)
        for app, r in (("gaussian", 2), ("sobel", 1)):
            with kp.Plan(app, W, H, r, "none", (0, 1), "nn", batch=B) as ex:
                ms_ex = time_kernel(lambda: ex.run(x, yex, stream), stream, steps, 3)
            out.append({"class": cls, "app": app, "r": r, "scheme": "none", "rate": [0, 1], "recon": "-",
                        "granule_bytes": None, "ms": ms_ex, "speedup": 1.0, "error": 0.0,
                        "hbm_gbs": 8 * px / ms_ex / 1e6})
            for scheme in ("row", "col", "checker"):
                for gb in ((128,) if scheme == "row" else (128, 4)):
                    for rate in ((1, 2), (1, 4), (3, 4)):
                        for recon in ("nn", "li"):
                            with kp.Plan(app, W, H, r, scheme, rate, recon, batch=B, granule_bytes=gb) as p:
                                ms = time_kernel(lambda: p.run(x, y, stream), stream, steps, 3)
                                err, _ = p.error(yex, y, stream)
                            k = 1.0 if gb == 4 else 1.0 - rate[0] / rate[1]  # G = 1 px: every 32-B sector is read
                            out.append({"class": cls, "app": app, "r": r, "scheme": scheme, "rate": list(rate),
                                        "recon": recon, "granule_bytes": gb, "ms": ms, "speedup": ms_ex / ms,
                                        "error": err, "hbm_gbs": bytes_per_px(app, scheme, rate) * px / ms / 1e6,
                                        "frac": bytes_per_px(app, scheme, rate) * px / ms / 1e6 / peak,
                                        "dram_bytes_floor_per_px": 4 * k + 4})
    return {"sweep": out, "workload": "C2 sweep: 8 x 4096^2 fp32 frames per class, seeds SEED_C2 + class",
            "metric": "ms per launch (CUDA events, 10 launches after 3 warm-up), speedup vs exact, error vs exact"}


def bench_hotspot(args, cfg, ws, rank, local, stream, peak, peak_src):
    import torch

    import paper_conf_cgo_maiercj18_b200 as kp
    import synth
    W, Hg, iters = cfg["W"], cfg["H"], cfg["iters"]
    # row bands: rank k owns rows [y0, y0 + h)
    cuts = kp.band_cuts(Hg, ws)
    y0, h = cuts[rank], cuts[rank + 1] - cuts[rank]
    T = torch.empty((h, W), device="cuda")
    P = torch.empty((h, W), device="cuda")
    synth.hotspot_band_device(cfg["seed"], W, Hg, y0, h, T.data_ptr(), P.data_ptr(), stream.cuda_stream)
    out = torch.empty_like(T)
    keys = dict(iters=iters, tblock=args.tblock)
    if ws > 1:
        keys.update(global_h=Hg, band_y0=y0)
    plan = kp.Plan("hotspot", W, h, 1, cfg["scheme"], cfg["rate"], cfg["recon"], **keys)
    exact = kp.Plan("hotspot", W, h, 1, "none", (0, 1), "nn", **keys)
    if ws > 1 and args.halo == "p2p":  # NEXT-4: peer stores + flags, handles swapped once
        import torch.distributed as dist
        for pl in (plan, exact):
            blobs = [None] * ws
            dist.all_gather_object(blobs, kp.perf_p2p_export(pl.handle))
            kp.perf_p2p_attach(pl.handle, blobs[rank - 1] if rank > 0 else None,
                               blobs[rank + 1] if rank < ws - 1 else None)
        barrier(ws)
    elif ws > 1:
        import torch.distributed as dist
        uid = kp.perf_comm_unique_id() if rank == 0 else bytes(128)
        t = torch.tensor(list(uid), dtype=torch.uint8, device="cuda" if dist.get_backend() == "nccl" else "cpu")
        dist.broadcast(t, 0)
        uid = bytes(t.cpu().tolist())
        kp.perf_comm_init(plan.handle, uid, rank, ws)
        kp.perf_comm_init(exact.handle, uid, rank, ws)
    run = lambda: plan.hotspot(T, P, out, stream)  # noqa: E731
    with ClockSampler(local) as clk:  # (warm-up inside: no idle gap before the timed steps)
        for _ in range(args.warmup):
            run()
        torch.cuda.synchronize()
        barrier(ws)
        e0 = torch.cuda.Event(enable_timing=True)
        e1 = torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        for _ in range(args.steps):
            run()
        e1.record(stream)
        e1.synchronize()
    barrier(ws)
    ms = max_over_ranks(ws, e0.elapsed_time(e1) / args.steps)
    out_ex = torch.empty_like(T)
    ms_ex = max_over_ranks(ws, time_kernel(lambda: exact.hotspot(T, P, out_ex, stream), stream, 2, 1))
    mre, cnt = plan.error(out_ex, out, stream)
    cells = W * Hg * iters
    # per launch: kept T + P read and T' written once; a launch covers tblock
    # steps under temporal blocking, one step otherwise
    algo_b = bytes_per_px("hotspot", cfg["scheme"], cfg["rate"]) * W * h * iters / max(args.tblock, 1)
    achieved = algo_b / (ms * 1e-3) / 1e9
    # NEXT-3 temporal blocking (single band only): TBLOCK steps per launch, T
    # perforated once per launch (R19) -- reported next to the
    # per-step headline, never in its place
    tblock = []
    if ws == 1 and not args.no_variants:
        for tb in (2, 4, 8):
            for sch, rt, rc in ((cfg["scheme"], cfg["rate"], cfg["recon"]), ("none", (0, 1), "nn")):
                q = kp.Plan("hotspot", W, h, 1, sch, rt, rc, iters=iters, tblock=tb)
                o2 = torch.empty_like(T)
                ms_tb = time_kernel(lambda: q.hotspot(T, P, o2, stream), stream, 3, 1)
                e_tb, _ = q.error(out_ex, o2, stream)
                tblock.append({"tblock": tb, "scheme": sch, "rate": list(rt), "recon": rc, "ms": ms_tb,
                               "mcell_s": cells / (ms_tb * 1e-3) / 1e6, "speedup_vs_exact_per_step": ms_ex / ms_tb,
                               "error_vs_exact_per_step": e_tb,
                               # kept T + P read and T' written once per launch of tb steps
                               "algorithmic_gbs": bytes_per_px("hotspot", sch, rt) * W * h * iters / tb
                               / (ms_tb * 1e-3) / 1e9})
                q.close()
    scratch = torch.empty((2, h, W), device="cuda")
    pmix = mixed_peak_gbs(scratch.data_ptr(), out_ex.data_ptr(), W * h * 4, cfg["scheme"], cfg["rate"], 128,
                          n_in=2, stream=stream.cuda_stream, pitch_bytes=W * 4)
    del scratch
    return {"metric": METRIC, "value": cells / (ms * 1e-3) / 1e6, "unit": "Mcell-updates/s", "n_gpus": ws,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True,
            "scaling": "strong", "vs_baseline": None, "dtype": "f32", "data": "synthetic",
            "config": {"workload": cfg["workload"] + (f", temporal blocking {args.tblock} steps/launch"
                                                      if args.tblock > 1 else ""),
                       "bands": ws, "tblock": args.tblock,
                       "halo": (("peer stores fused into the step kernel + epoch flags (NEXT-4)"
                                 if args.halo == "p2p" else "NCCL send/recv per launch") if ws > 1 else "none")},
            "speedup_vs_exact": ms_ex / ms, "error": {"metric": "mre", "value": mre, "count": cnt},
            "roofline": {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s",
                         "frac": achieved / peak,
                         # per-step launch on one GPU (tools/ncu_traffic.py); blocked / banded runs: none captured
                         "traffic": ncu_traffic("C4", f"hotspot1_{cfg['scheme']}_{cfg['rate'][0]}-{cfg['rate'][1]}_"
                                                      f"{cfg['recon']}") if ws == 1 and args.tblock == 1 else None,
                         "kernel": "hotspot per-step launch" if args.tblock == 1 else "hotspot_tb_kernel",
                         "algorithmic_bytes_per_launch": algo_b / max(1, -(-iters // max(args.tblock, 1))),
                         "peak_source": peak_src,
                         "peak_mix": pmix, "frac_mix": achieved / pmix if pmix else None},
            # our kernels per timed call: one per launch of TBLOCK steps; banded runs split each launch into
            # boundary rows (2 launches) + interior (PERF_KEY_OVERLAP), peer-store runs add signal + wait kernels
            "clocks": clk.summary(), "gpu_launches": args.steps * (-(-iters // args.tblock)) * (3 if ws > 1 else 1),
            "temporal_blocking": tblock}


if __name__ == "__main__":
    main()
