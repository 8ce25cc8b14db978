#!/usr/bin/env python
"""Benchmark of the hot path (BASELINE.json metric: "Dslash GFLOPS & HBM GB/s per B200 at
1/2/4/8 GPUs; mixed-prec solve time").

Workload (BASELINE.json configs[4], the weak-scaling configuration that fits one GPU and is
defined at every GPU count): 32^3 x 64 sites per GPU, global lattice 32^3 x (64 N),
T-partitioned across N ranks.  Weak-field SU(3) gauge (eps = 0.1),
kappa = 0.124, c_sw = 1.0, antiperiodic T.

One STEP = one mixed-precision reliable-update BiCGstab solve of a fixed ITERS iterations
(tol = 0, delta = 1e-3; fp64 outer with fp64 18-real links, fp32 sloppy with 12-real links),
through the C-ABI entry qudax_solve_bicgstab_dev: Schur prepare, ITERS x (2 Mhat = 4 Dslash
kernels + 4 halo exchanges, 5 fused BLAS kernels, 3 global reductions), the fp64 reliable
updates, reconstruction and the fp64 true residual — every row of SURVEY §8(a) except the
once-per-configuration setup (gauge upload, clover build).  value = effective flops
(P:755-758 convention: 3696 per even site per Mhat + 960 BLAS, reading Q16) of all ranks /
max-over-ranks device time.

Run:   python bench.py [--gpus N --steps K --warmup W]
       torchrun --nproc-per-node N bench.py --gpus N ...
       python bench.py --impl reference      (the fp64 CPU oracle on the host cores)
"""
import argparse
import json
import os
import statistics
import subprocess
import sys
import tempfile
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)
# NCCL's graph-mixing support adds an external event-wait node to every NCCL operation captured
# in a graph, which a conditional (WHILE) graph body cannot hold: with it, a partitioned solve
# falls back to one host poll per iteration (the library prints why).  The library never runs
# graph-captured and eager NCCL work of one communicator concurrently, so the bench (the NCCL
# user of this process) switches it off before NCCL initialises (profiles/r02ab_*).
os.environ.setdefault("NCCL_GRAPH_MIXING_SUPPORT", "0")

METRIC = "Dslash GFLOPS & HBM GB/s per B200 at 1/2/4/8 GPUs; mixed-prec solve time"
KAPPA, CSW, EPS = 0.124, 1.0, 0.1
# reliable-update thresholds (reading Q11): double-half the paper's 1e-2
# (P:787-790); double-single (not given) the paper's single-precision 1e-3
DELTA_DS, DELTA_DH = 1e-3, 1e-2
SPATIAL, T_PER_GPU, T_STRONG = 32, 64, 256
GAUGE_SEED, SRC_SEED = 1005, 2005
BLAS_FLOPS_PER_SITE_ITER = 960.0


def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--iters", type=int, default=100, help="BiCGstab iterations per step")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-extra", action="store_true", help="skip the per-precision Dslash table and the config-3 solve")
    ap.add_argument("--overlap", type=int, default=1)
    ap.add_argument("--halo", default="comm", choices=["comm", "p2p"],
                    help="N>1 spinor halo: NCCL send/recv (comm) or kernel-initiated over peer memory (p2p)")
    ap.add_argument("--grid", default="", help="process grid Px,Py,Pz,Pt (default 1,1,1,N: T slabs, P:563-605; "
                                               "others: multi-dimensional split, SURVEY 8(f) item 4)")
    ap.add_argument("--no-kernel-timing", action="store_true",
                    help="diagnostic: no per-launch CUDA events in the timed region (no roofline)")
    ap.add_argument("--breakdown", action="store_true",
                    help="diagnostic: per (precision, kind, fused reduction) in-step Dslash times to stderr")
    ap.add_argument("--scaling", default="weak", choices=["weak", "strong"],
                    help="weak: 32^3x64 per GPU (BASELINE configs[4]); strong: 32^3x256 in total (configs[3])")
    ap.add_argument("--oracle-sample", type=int, default=0, help=argparse.SUPPRESS)  # internal: 1-thread oracle run
    ap.add_argument("--oracle-ops", action="store_true", help=argparse.SUPPRESS)  # internal: 1-thread oracle ops
    return ap.parse_args()


def cpu_oracle_1thread(iters=2):
    """The same oracle sample on ONE host thread (oracle timed with nproc threads
    and with 1), in a child process: OpenMP fixes its thread count at first use."""
    import subprocess
    env = dict(os.environ, OMP_NUM_THREADS="1")
    r = subprocess.run([sys.executable, os.path.abspath(__file__), "--oracle-sample", str(iters)], env=env,
                       capture_output=True, text=True, timeout=600)
    if r.returncode != 0:
        return None
    return json.loads(r.stdout.strip().splitlines()[-1])


# ---------------------------------------------------------------------------- clocks
class ClockSampler:
    """nvidia-smi clocks and throttle reasons sampled every 200 ms during the timed region."""
    FIELDS = "index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.hw_slowdown," \
             "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown," \
             "clocks_event_reasons.sw_power_cap"

    def __init__(self, device):
        self.device = device
        self.proc = None
        self.path = None

    def __enter__(self):
        try:
            fd, self.path = tempfile.mkstemp(suffix=".csv")
            os.close(fd)
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.device), f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                 "-lms", "200"], stdout=open(self.path, "w"), stderr=subprocess.DEVNULL)
        except Exception:  # noqa: BLE001
            self.proc = None
        return self

    def __exit__(self, *a):
        if self.proc is not None:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except Exception:  # noqa: BLE001
                self.proc.kill()

    def summary(self):
        if not self.path or not os.path.exists(self.path):
            return None
        rows = []
        for line in open(self.path):
            parts = [p.strip() for p in line.split(",")]
            if len(parts) < 8:
                continue
            try:
                rows.append((float(parts[1]), float(parts[2]), parts[4:8]))
            except ValueError:
                continue
        os.unlink(self.path)
        if not rows:
            return None
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[k] for _, _, r in rows for k in range(4) if r[k].lower() == "active"})
        sm_max = max(r[1] for r in rows)
        loaded = [r[0] for r in rows if r[0] > 0.3 * sm_max] or [r[0] for r in rows]
        return {"sm_mhz": statistics.median(loaded), "sm_max_mhz": sm_max, "reasons": reasons, "samples": len(rows)}


# ---------------------------------------------------------------------------- helpers
def measured_peak():
    path = os.path.join(ROOT, "MEASURED_PEAKS.json")
    try:
        d = json.load(open(path))
        return float(d["hbm_gbs"]), "MEASURED_PEAKS.json hbm_gbs (STREAM-style copy, of measured)"
    except Exception:  # noqa: BLE001
        return 6650.0, "B200_PROFILING.md fallback 6.65 TB/s (of fallback)"


def profiled_traffic():
    """dram bytes per Dslash launch from the committed ncu --set full summary (or None)."""
    path = os.path.join(ROOT, "profiles", "dslash_traffic.json")
    try:
        d = json.load(open(path))
        return d
    except Exception:  # noqa: BLE001
        return None


def cpu_oracle_gflops(iters, dims=(SPATIAL, SPATIAL, SPATIAL, 8)):
    """The fp64 oracle (oracle/, as it stands) on a bounded sample: `iters` textbook BiCGstab
    iterations on Mhat of a 32^3 x 8 lattice of the same kind (weak field, same kappa/c_sw).
    Returns (gflops, seconds, threads, sample description)."""
    import numpy as np

    import oracle
    import qgen
    U = qgen.gauge(dims, GAUGE_SEED, eps=EPS)
    wc = oracle.WilsonClover(U, KAPPA, CSW, -1.0)
    b = oracle.restrict(qgen.spinor(dims, SRC_SEED), 0)
    t0 = time.perf_counter()
    oracle.bicgstab(wc.matpc, b, tol=0.0, maxiter=iters)
    dt = time.perf_counter() - t0
    vh = np.prod(dims) / 2
    flops = iters * (2 * 3696 + BLAS_FLOPS_PER_SITE_ITER) * vh
    threads = int(os.environ.get("OMP_NUM_THREADS", os.cpu_count() or 1))
    sample = f"{iters} oracle BiCGstab iterations on Mhat of a {dims[0]}^3x{dims[3]} weak-field lattice (fp64, C+OpenMP+numpy)"
    return flops / dt * 1e-9, dt, threads, sample


def single_gpu_extras(ctx, b_dev, peak):
    """N = 1 only: multi-RHS Mhat (fp32-12, 4 and 8 RHS) on the bench lattice, and the
    half-precision (recon 12) Mhat in a second context.  Per-launch CUDA-event timing."""
    from paper_1011_0024_b200 import qudax
    out = {}
    fin = ctx.new_field(4)
    ctx.spinor_load_dev(fin, 4, 0, b_dev)
    for n in (4, 8):
        ins = [fin] * n
        outs = [ctx.new_field(4) for _ in range(n)]
        for _ in range(3):
            ctx.matpc_multi(outs, ins, 4)
        ctx.kernel_timing(True)
        for _ in range(10):
            ctx.matpc_multi(outs, ins, 4)
        ks = ctx.kernel_stats(prec=4)
        ctx.kernel_timing(False)
        gbs = ks["bytes_compulsory"] / (ks["ms_total"] * 1e-3) * 1e-9
        out[f"fp32-12 x{n} rhs"] = {"matpc_gflops": ks["flops"] / (ks["ms_total"] * 1e-3) * 1e-9,
                                   "us_per_rhs": 1e3 * ks["ms_total"] / 10 / n,
                                   "gbs_multi_rhs_model": gbs, "frac_of_measured_hbm": gbs / peak}
    import numpy as np
    import qgen
    dims = ctx.global_dims
    hctx = qudax.Context(dims)
    hctx.gauge_load(qgen.gauge(dims, GAUGE_SEED, eps=EPS), KAPPA, CSW, prec=2, recon=12)
    hi, ho = hctx.new_field(2), hctx.new_field(2)
    hctx.spinor_load_dev(hi, 2, 0, b_dev)
    for _ in range(3):
        hctx.matpc(ho, hi, 2)
    hctx.kernel_timing(True)
    for _ in range(30):
        hctx.matpc(ho, hi, 2)
    ks = hctx.kernel_stats(prec=2)
    hctx.close()
    gbs = ks["bytes_compulsory"] / (ks["ms_total"] * 1e-3) * 1e-9
    out["half-12"] = {"kernel_gflops": ks["flops"] / (ks["ms_total"] * 1e-3) * 1e-9, "kernel_gbs_compulsory": gbs,
                      "frac_of_measured_hbm": gbs / peak, "matpc_us": 1e3 * ks["ms_total"] / 30}
    del np
    return out


def oracle_operator_seconds(reps=1):
    """SURVEY 8(d) timing protocol: the fp64 oracle's seconds per Dslash (eq. 2, all sites) and
    per Mhat (even sites), on the box's host cores, for BASELINE configs[0..2] (4^4, 16^3x32,
    24^3x128).  Returns {config: {"dslash_s", "matpc_s", "threads"}}; run once with the default
    OpenMP thread count and once in a child with OMP_NUM_THREADS=1 (oracle_operator_seconds_1thread)."""
    import numpy as np

    import oracle
    import qgen
    out = {}
    oracle.dslash(qgen.gauge((4, 4, 4, 4), 1), qgen.spinor((4, 4, 4, 4), 2))  # OpenMP thread start-up
    for name, dims, gseed in (("configs[0] 4^4", (4, 4, 4, 4), 1001), ("configs[1] 16^3x32", (16, 16, 16, 32), 1002),
                              ("configs[2] 24^3x128", (24, 24, 24, 128), 1003)):
        U = qgen.gauge(dims, gseed, eps=-1.0 if gseed != 1003 else EPS)
        psi = qgen.spinor(dims, gseed + 1000)
        t0 = time.perf_counter()
        for _ in range(reps):
            oracle.dslash(U, psi, -1.0)
        t_d = (time.perf_counter() - t0) / reps
        wc = oracle.WilsonClover(U, KAPPA, CSW, -1.0)
        pe = oracle.restrict(psi, 0)
        t0 = time.perf_counter()
        for _ in range(reps):
            wc.matpc(pe)
        t_m = (time.perf_counter() - t0) / reps
        vh = np.prod(dims) / 2
        out[name] = {"dslash_s": t_d, "matpc_s": t_m, "dslash_gflops": 1320 * 2 * vh / t_d * 1e-9,
                     "matpc_gflops": 3696 * vh / t_m * 1e-9}
        del U, psi, wc, pe
    threads = int(os.environ.get("OMP_NUM_THREADS", os.cpu_count() or 1))
    return {"threads": threads, "configs": out,
            "note": "oracle = plain fp64 C (OpenMP) + numpy; Dslash over every site of the lattice, Mhat on the even "
                    "sites (clover build excluded, done once per WilsonClover)"}


def oracle_operator_seconds_1thread():
    env = dict(os.environ, OMP_NUM_THREADS="1")
    r = subprocess.run([sys.executable, os.path.abspath(__file__), "--oracle-ops"], env=env, capture_output=True,
                       text=True, timeout=900)
    if r.returncode != 0:
        return None
    return json.loads(r.stdout.strip().splitlines()[-1])


def config2_l2_resident(peak):
    """BASELINE configs[1]: 16^3x32 (fp32-12, 57 MB working set < the 126 MB L2): Mhat timed
    back to back — the number is L2-RESIDENT, labelled so, not an HBM measurement."""
    import torch

    import qgen
    from paper_1011_0024_b200 import qudax
    dims = (16, 16, 16, 32)
    ctx = qudax.Context(dims)
    ctx.gauge_load(qgen.gauge(dims, 1002), 0.12, 1.0, prec=4, recon=12)
    fi, fo = ctx.new_field(4), ctx.new_field(4)
    ctx.spinor_load(fi, 4, 0, qgen.spinor(dims, 2002))
    times = timed_reps(ctx, lambda: ctx.matpc(fo, fi, 4), 60)
    ctx.close()
    m = qudax.site_model(4, 12, -1)
    vh = 16 ** 3 * 32 // 2
    med = statistics.median(times)
    return {"lattice": "16^3x32 fp32-12 Mhat", "l2_resident": True, "matpc_us_median": 1e3 * med,
            "matpc_us_min": 1e3 * min(times), "reps": len(times),
            "matpc_gflops_median": m["flops"] * vh / (med * 1e-3) * 1e-9,
            "model_gbs_median": m["bytes_compulsory"] * vh / (med * 1e-3) * 1e-9,
            "note": "working set ~57 MB < 126 MB L2: L2-resident bandwidth, not HBM"}


def timed_reps(ctx, fn, reps, warm=5):
    """Per-application times (ms) of `fn` on the context's stream: CUDA events around each of
    `reps` back-to-back applications after `warm` untimed ones (SURVEY 8(d) timing protocol)."""
    import torch
    for _ in range(warm):
        fn()
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(reps + 1)]
    ev[0].record(ctx.stream)
    for k in range(reps):
        fn()
        ev[k + 1].record(ctx.stream)
    ctx.stream.synchronize()
    return [ev[k].elapsed_time(ev[k + 1]) for k in range(reps)]


def config3_solve_time():
    """BASELINE configs[2]: 24^3 x 128 weak field, the paper's 6 point sources (colour 0-2 x
    spin 0-1), mixed double-single (delta 1e-3, the paper's single-precision value;
    DESIGN.md reading Q11) and double-half (delta 1e-2, the paper's value)
    reliable-update BiCGstab to ||r||/||b|| <= 1e-14 through the C-ABI
    with host buffers; mean time to solution, iterations, true residual."""
    import qgen
    from paper_1011_0024_b200 import qudax
    dims = (24, 24, 24, 128)
    U = qgen.gauge(dims, 1003, eps=EPS)
    ctx = qudax.Context(dims)
    res = {"workload": "24^3x128 weak field, 6 point sources, tol 1e-14, kappa 0.124, csw 1.0 (BASELINE configs[2])"}
    for name, ps, delta in (("double-single", 4, DELTA_DS), ("double-half", 2, DELTA_DH)):
        ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=ps, recon_sloppy=12, t_boundary=-1)
        srcs = [qgen.point_source(dims, spin, colour) for colour in range(3) for spin in range(2)]
        # warm-up (workspace allocation, graph capture) outside the timed solves, for both forms
        ctx.solve(srcs[0], tol=0, delta=delta, maxiter=3, prec=8, prec_sloppy=ps, allow_not_converged=True)
        ctx.solve_multi(srcs, tol=0, delta=delta, maxiter=3, prec=8, prec_sloppy=ps, allow_not_converged=True)
        ts, its, trs, gfl = [], [], [], []
        for colour in range(3):
            for spin in range(2):
                b = qgen.point_source(dims, spin, colour)
                _, st = ctx.solve(b, tol=1e-14, delta=delta, maxiter=20000, prec=8, prec_sloppy=ps,
                                  allow_not_converged=True)
                ts.append(st["secs"])
                its.append(st["iters"])
                trs.append(st["true_res"])
                gfl.append(st["gflops"])
        res[name] = {"mean_secs": sum(ts) / len(ts), "mean_iters": sum(its) / len(its), "max_true_res": max(trs),
                     "mean_gflops": sum(gfl) / len(gfl)}
        # the same 6 sources as ONE batched solve (multi-RHS Mhat, per-system fused reductions):
        # seconds per source = batch wall time / 6
        _, sts = ctx.solve_multi(srcs, tol=1e-14, delta=delta, maxiter=20000, prec=8, prec_sloppy=ps,
                                 allow_not_converged=True)
        secs = sts[0]["secs"]
        res[name + " batched x6"] = {"secs_per_source": secs / len(srcs), "batch_secs": secs,
                                     "mean_iters": sum(s["iters"] for s in sts) / len(sts),
                                     "max_true_res": max(s["true_res"] for s in sts),
                                     "gflops": sum(s["flops"] for s in sts) / secs * 1e-9}
    ctx.close()
    return res


# ---------------------------------------------------------------------------- reference arm
def run_reference(args):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return
    K, W = args.steps, args.warmup
    iters = 2
    for _ in range(W):
        cpu_oracle_gflops(1)
    times, gfl = [], []
    for _ in range(K):
        g, dt, threads, sample = cpu_oracle_gflops(iters)
        times.append(dt)
        gfl.append(g)
    value = sum(gfl) / len(gfl)
    out = {
        "impl": "reference", "metric": METRIC, "value": value, "unit": "GFLOPS", "n_gpus": args.gpus,
        "steps": K, "warmup": W, "ms_per_step": 1e3 * sum(times) / len(times), "higher_is_better": True,
        "scaling": "weak", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
        "config": {"workload": "oracle sample of the weak-scaling 32^3x64-per-GPU BiCGstab workload",
                   "sample": sample},
        "cpu_baseline": {"value": value, "unit": "GFLOPS", "cores": threads, "kind": "oracle", "sample": sample},
        "e2e": {"value": value, "unit": "GFLOPS", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(out))


# ---------------------------------------------------------------------------- our arm
def main():
    if "--oracle-ops" in sys.argv:  # child of oracle_operator_seconds_1thread (no GPU work)
        print(json.dumps(oracle_operator_seconds()))
        return
    if "--oracle-sample" in sys.argv:  # child of cpu_oracle_1thread (no GPU work)
        a = parse()
        g, dt, threads, sample = cpu_oracle_gflops(a.oracle_sample)
        print(json.dumps({"value": g, "seconds": dt, "cores": threads, "sample": sample}))
        return
    args = parse()
    if args.impl == "reference":
        return run_reference(args)
    import numpy as np
    import torch
    import torch.distributed as dist

    import qgen
    from paper_1011_0024_b200 import qudax

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    N = world
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if world > 1:
        dist.init_process_group("nccl", device_id=dev)
    grid = tuple(int(v) for v in args.grid.split(",")) if args.grid else (1, 1, 1, N)
    assert len(grid) == 4 and grid[0] * grid[1] * grid[2] * grid[3] == N, "grid must multiply to the GPU count"
    if args.scaling == "weak":
        local_dims = (SPATIAL, SPATIAL, SPATIAL, T_PER_GPU)
        dims = tuple(l * p for l, p in zip(local_dims, grid))
    else:
        dims = (SPATIAL, SPATIAL, SPATIAL, T_STRONG)
        local_dims = tuple(d // p for d, p in zip(dims, grid))
    T_loc = local_dims[3]

    def barrier():
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()

    def max_over_ranks(v):
        if world == 1:
            return v
        t = torch.tensor([v], dtype=torch.float64, device=dev)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        return float(t.item())

    # ---- context + setup (once per configuration, not timed)
    if world > 1:
        obj = [qudax.nccl_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        obj2 = [qudax.nccl_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj2, src=0)
        ctx = qudax.Context(dims, nranks=N, rank=rank, device=local, comm=qudax.COMM_NCCL, nccl_id=obj[0],
                            overlap=bool(args.overlap), proc_grid=grid,
                            halo=qudax.HALO_P2P if args.halo == "p2p" else qudax.HALO_COMM)
    else:
        ctx = qudax.Context(dims, device=local, flags=qudax.FLAG_TIMING_BREAKDOWN if args.breakdown else 0)
    assert ctx.local_dims == local_dims, (ctx.local_dims, local_dims)
    origin = ctx.partition["origin"]
    U = qgen.gauge_box(dims, GAUGE_SEED, origin, local_dims, eps=EPS)
    ctx.gauge_load(U, KAPPA, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12, t_boundary=-1)
    del U
    b_host = qgen.spinor_box(dims, SRC_SEED, origin, local_dims)
    with torch.cuda.stream(ctx.stream):
        b_dev = torch.from_numpy(b_host.view(np.float64)).to(dev)
        x_dev = torch.zeros_like(b_dev)
    ctx.stream.synchronize()
    b_pin = torch.from_numpy(b_host.view(np.float64)).pin_memory()
    x_pin = torch.zeros_like(b_pin).pin_memory()
    solve_kw = dict(tol=0.0, delta=DELTA_DS, maxiter=args.iters, prec=8, prec_sloppy=4, allow_not_converged=True)

    # ---- warm-up
    for _ in range(args.warmup):
        ctx.solve_dev(x_dev, b_dev, **solve_kw)
    barrier()

    # ---- timed region (device-resident inputs).  Pass 1 gives `value`: no per-launch events
    # (inside graph replay each event-record node costs ~5 us of launch pipelining: measured
    # 95.0 vs 99.2 ms per step, gpurun r02d).  Pass 2 repeats the same K steps with CUDA events
    # around every Dslash launch on the launching stream and gives the roofline.
    def timed_pass(events, span=False):
        l0 = ctx.launch_count()
        ctx.kernel_timing(events, span=span)
        fl, it, up = 0.0, 0, 0
        with ClockSampler(local) as clk:
            barrier()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(ctx.stream)
            for _ in range(args.steps):
                st = ctx.solve_dev(x_dev, b_dev, **solve_kw)
                fl += st["flops"]
                it += st["iters"]
                up += st["reliable_updates"]
            e1.record(ctx.stream)
            barrier()
        t = max_over_ranks(e0.elapsed_time(e1))
        kst = ctx.kernel_stats(prec=4) if events else None  # the sloppy fp32 recon-12 Dslash
        ctx.kernel_timing(False)
        return t, fl, it, up, ctx.launch_count() - l0, kst, clk.summary()

    ms, flops, iters, updates, launches, _, clocks = timed_pass(False)
    value = flops / (ms * 1e-3) * 1e-9  # flops already counts all ranks' sites
    ks = {"ms_total": 0.0, "launches": 0, "bytes_compulsory": 0.0, "flops": 0.0, "bytes_paper": 0.0}
    ms_ev = None
    ks_span = None
    if not args.no_kernel_timing:
        ms_ev, _, _, _, _, ks, _ = timed_pass(True)
        # pass 3: the in-kernel span of the same launches (its stamps cost the kernels a few us,
        # so it does not share the events pass)
        _, _, _, _, _, ks_span, _ = timed_pass(True, span=True)

    # ---- roofline of the dominant kernel (the Dslash, fp32 12-reconstruct, both kinds)
    peak, peak_src = measured_peak()
    avg_ms = ks["ms_total"] / max(ks["launches"], 1)
    achieved = ks["bytes_compulsory"] / (ks["ms_total"] * 1e-3) * 1e-9 if ks["ms_total"] > 0 else 0.0
    trafficd = profiled_traffic()
    traffic = None
    if trafficd and trafficd.get("lattice") == list(local_dims):
        traffic = trafficd.get("dram_bytes_per_launch")
    roofline = {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s", "frac": achieved / peak,
                "traffic": traffic, "kernel": "dslash_kernel fp32 recon-12 (clover-inverse + clover-xpay kinds)",
                "bytes_model": "compulsory (SURVEY 8(d)): 864 B/site clover-inv, 960 B/site xpay",
                "avg_launch_ms": avg_ms, "launches": ks["launches"], "peak_source": peak_src,
                "kernel_gflops": ks["flops"] / (ks["ms_total"] * 1e-3) * 1e-9 if ks["ms_total"] > 0 else 0.0,
                "paper_model_gbs": ks["bytes_paper"] / (ks["ms_total"] * 1e-3) * 1e-9 if ks["ms_total"] > 0 else 0.0,
                "kernel_share_of_step": ks["ms_total"] / ms_ev if ms_ev else None,
                "kernel_span": ({"avg_span_ms": ks_span["span_ms_total"] / max(ks_span["launches"], 1),
                                 "achieved_gbs": ks_span["bytes_compulsory"] / (ks_span["span_ms_total"] * 1e-3) * 1e-9,
                                 "frac": ks_span["bytes_compulsory"] / (ks_span["span_ms_total"] * 1e-3) * 1e-9 / peak,
                                 "note": "pass 3, the same K steps: %globaltimer from the first CTA's start to the last "
                                         "CTA's end inside each kernel (no event-node launch bubble; the stamps "
                                         "themselves cost a few us per launch)"}
                                if ks_span and ks_span.get("span_ms_total") else None),
                "timed_region": (f"second pass of the same {args.steps} steps with CUDA events around every Dslash "
                                 f"launch ({ms_ev / args.steps:.2f} ms per step with the events, "
                                 f"{ms / args.steps:.2f} ms without: value)") if ms_ev else None}

    # ---- end to end through the C-ABI with pinned host buffers (H2D of b, D2H of x inside)
    barrier()
    e2 = [torch.cuda.Event(enable_timing=True) for _ in range(2)]
    flops_e2e = 0.0
    e2[0].record(ctx.stream)
    for _ in range(args.steps):
        _, st = ctx.solve(b_pin, out=x_pin, **solve_kw)
        flops_e2e += st["flops"]
    e2[1].record(ctx.stream)
    barrier()
    ms_e2e = max_over_ranks(e2[0].elapsed_time(e2[1]))
    nbytes = b_pin.numel() * 8
    e2e = {"value": flops_e2e / (ms_e2e * 1e-3) * 1e-9, "unit": "GFLOPS", "h2d_bytes_per_step": nbytes,
           "d2h_bytes_per_step": nbytes, "api": "qudax_solve_bicgstab (host buffers, pinned)"}

    # ---- Dslash-only numbers (Mhat applications, device resident), per precision
    dslash = {}
    vh_loc = local_dims[0] * local_dims[1] * local_dims[2] * T_loc // 2

    def matpc_numbers(c, prec, recon, reps=50):
        """Mhat applied `reps` times back to back: per-application CUDA-event times (median and
        minimum, max over ranks of each), plus the Dslash kernels' own event times."""
        fin, fout = c.new_field(prec), c.new_field(prec)
        c.spinor_load_dev(fin, prec, 0, b_dev)
        barrier()
        c.kernel_timing(True)
        times = timed_reps(c, lambda: c.matpc(fout, fin, prec), reps)
        k2 = c.kernel_stats(prec=prec)
        c.kernel_timing(False)
        barrier()
        med, mn = max_over_ranks(statistics.median(times)), max_over_ranks(min(times))
        m = qudax.site_model(prec, recon, -1)
        kg = k2["bytes_compulsory"] / (k2["ms_total"] * 1e-3) * 1e-9
        return {"matpc_us_median": 1e3 * med, "matpc_us_min": 1e3 * mn, "reps": reps,
                "matpc_gflops_total": m["flops"] * vh_loc * N / (med * 1e-3) * 1e-9,
                "matpc_gflops_per_gpu": m["flops"] * vh_loc / (med * 1e-3) * 1e-9,
                "model_gbs_per_gpu": m["bytes_compulsory"] * vh_loc / (med * 1e-3) * 1e-9,
                "kernel_gbs_compulsory": kg, "kernel_gflops": k2["flops"] / (k2["ms_total"] * 1e-3) * 1e-9,
                "frac_of_measured_hbm": kg / peak}

    if not args.no_extra:
        for prec, recon, name in ((4, 12, "fp32-12"), (8, 18, "fp64-18")):
            dslash[name] = matpc_numbers(ctx, prec, recon)
        # the paper's "solver runs 10-20% slower than the matvec": one BiCGstab
        # iteration (2 Mhat + BLAS) of the timed solves against 2 bare Mhat applications
        it_ms = ms / max(iters, 1)
        dslash["solver_vs_matpc"] = {"iteration_ms": it_ms, "two_matpc_ms": 2e-3 * dslash["fp32-12"]["matpc_us_median"],
                                     "solver_slower_by": it_ms / (2e-3 * dslash["fp32-12"]["matpc_us_median"]) - 1,
                                     "note": "step time incl. reliable updates, Schur prepare/reconstruct and the "
                                             "final fp64 residual, per iteration"}
        if N > 1:
            # weak-scaling reference on the same box: each rank's local lattice on ONE GPU through the
            # unsplit (no-communication) path, and the split path with the overlap switched off
            one = qudax.Context(local_dims, device=local)
            one.gauge_load(qgen.gauge(local_dims, GAUGE_SEED, eps=EPS), KAPPA, CSW, prec=4, recon=12, t_boundary=-1)
            n1 = matpc_numbers(one, 4, 12)
            one.close()
            dslash["weak_scaling_fp32-12"] = {
                "matpc_gflops_N": dslash["fp32-12"]["matpc_gflops_total"],
                "matpc_gflops_1gpu_unsplit": n1["matpc_gflops_per_gpu"],
                "efficiency": dslash["fp32-12"]["matpc_gflops_total"] / (N * n1["matpc_gflops_per_gpu"]),
                "note": "GFLOPS_N / (N x GFLOPS_1), 1-GPU baseline = the unsplit kernel on the per-GPU lattice"}
            if args.halo == "comm":
                nov = qudax.Context(dims, nranks=N, rank=rank, device=local, comm=qudax.COMM_NCCL,
                                    nccl_id=obj2[0], overlap=False, proc_grid=grid)
                Ub = qgen.gauge_box(dims, GAUGE_SEED, origin, local_dims, eps=EPS)
                nov.gauge_load(Ub, KAPPA, CSW, prec=4, recon=12, t_boundary=-1)
                del Ub
                dslash["fp32-12 overlap off"] = matpc_numbers(nov, 4, 12)
                nov.close()
    solve_time = None
    if not args.no_extra and N == 1:
        dslash.update(single_gpu_extras(ctx, b_dev, peak))
        dslash["config2 L2-resident"] = config2_l2_resident(peak)
        solve_time = config3_solve_time()

    # ---- CPU baseline: the oracle on the host cores (rank 0, N = 1 only)
    cpu = None
    if rank == 0 and N == 1 and not args.no_cpu_baseline:
        g, dt, threads, sample = cpu_oracle_gflops(20)
        cpu = {"value": g, "unit": "GFLOPS", "cores": threads, "kind": "oracle", "sample": sample, "seconds": dt}
        one = cpu_oracle_1thread(2)
        if one:
            cpu["one_thread"] = {"value": one["value"], "cores": one["cores"], "sample": one["sample"],
                                 "seconds": one["seconds"]}
        if not args.no_extra:
            cpu["oracle_operators"] = oracle_operator_seconds()
            cpu["oracle_operators_1thread"] = oracle_operator_seconds_1thread()

    ctx.close()
    if rank == 0:
        out = {
            "metric": METRIC, "value": value, "unit": "GFLOPS", "n_gpus": N, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": ms / args.steps, "higher_is_better": True, "scaling": args.scaling,
            "vs_baseline": None, "dtype": "f32", "data": "synthetic",
            "config": {"workload": (f"weak scaling 32^3x64 per GPU (global {'x'.join(map(str, dims))}), "
                                    if args.scaling == "weak" else
                                    f"strong scaling 32^3x256 in total ({'x'.join(map(str, local_dims))} per GPU), ")
                                   + f"mixed-precision reliable-update BiCGstab, {args.iters} iterations per step "
                                   + ("(BASELINE configs[4])" if args.scaling == "weak" else "(BASELINE configs[3])"),
                       "lattice_global": list(dims), "lattice_per_gpu": list(local_dims), "proc_grid": list(grid),
                       "precision": {"outer": "f64 recon-18", "sloppy": "f32 recon-12"},
                       "kappa": KAPPA, "csw": CSW, "gauge": f"weak field eps={EPS}", "t_boundary": "antiperiodic",
                       "delta": DELTA_DS, "parallelism": ("grid " + "x".join(map(str, grid)) if args.grid else f"T-slab x{N}")
                                                    + ((" (P2P kernel-initiated halo)" if args.halo == "p2p" else
                                                        " (NCCL halo, overlapped)") if N > 1 else ""),
                       "l2": "inputs larger than L2 (>1 GB of gauge+clover+fields per GPU vs 126 MB L2)"},
            "iters_per_step": iters / args.steps, "reliable_updates_per_step": updates / args.steps,
            "roofline": roofline, "cpu_baseline": cpu, "e2e": e2e, "gpu_launches": launches, "clocks": clocks,
            "dslash": dslash, "solve_time": solve_time,
        }
        print(json.dumps(out))
    if world > 1:
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
