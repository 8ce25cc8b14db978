"""Multi-rank worker (launched by tests/gpu/test_multirank.py through torchrun).

Every rank drives one qudax context on ITS box of a global lattice split over a process grid
(default T slabs; --grid Px,Py,Pz,Pt for the multi-dimensional split).  All ranks
may share one GPU (the QUDAX_COMM_HOST transport stages faces through pinned host memory and
exchanges them with torch.distributed/gloo — the paper's non-overlapped strategy),
or use NCCL when the ranks own distinct GPUs.  Rank 0 gathers the slabs and compares them
BITWISE with the unpartitioned single-context result (the exchange moves bits only), and the
solver's solution with the fp64 oracle.

    torchrun --nproc-per-node N tests/gpu/mp_worker.py --comm host|nccl --out result.json
"""
import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--comm", default="host")
    ap.add_argument("--out", required=True)
    ap.add_argument("--dims", default="8,4,6,16")
    ap.add_argument("--same-gpu", type=int, default=1)
    ap.add_argument("--halo", default="comm", help="comm | p2p (kernel-initiated over CUDA IPC peer memory)")
    ap.add_argument("--grid", default="", help="process grid Px,Py,Pz,Pt (default 1,1,1,N: T slabs)")
    args = ap.parse_args()
    dims = tuple(int(v) for v in args.dims.split(","))
    dist.init_process_group("gloo")
    rank, n = dist.get_rank(), dist.get_world_size()
    device = 0 if args.same_gpu else rank
    torch.cuda.set_device(device)
    grid = tuple(int(v) for v in args.grid.split(",")) if args.grid else (1, 1, 1, n)
    part = qudax.partition_info(dims, n, rank, proc_grid=grid)
    L, o = part["local_dims"], part["origin"]

    def box(a, lead=0):
        """this rank's box of a global [.., T, Z, Y, X, ...] array (lead = leading axes)"""
        sl = (slice(None),) * lead + tuple(slice(o[m], o[m] + L[m]) for m in (3, 2, 1, 0))
        return np.ascontiguousarray(a[sl])
    Ug_all = qgen.gauge(dims, 1301, eps=-1.0)
    U = box(Ug_all, 1)
    psi = box(qgen.spinor(dims, 1302))
    xin = box(qgen.spinor(dims, 1303))
    result = {"rank": rank, "n": n, "comm": args.comm, "halo": args.halo, "grid": grid, "ok": True, "checks": {}}
    halo = qudax.HALO_P2P if args.halo == "p2p" else qudax.HALO_COMM
    if args.comm == "nccl":
        obj = [qudax.nccl_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        ctx = qudax.Context(dims, nranks=n, rank=rank, device=device, comm=qudax.COMM_NCCL, nccl_id=obj[0],
                            halo=halo, proc_grid=grid)
    else:
        ctx = qudax.Context(dims, nranks=n, rank=rank, device=device, comm=qudax.COMM_HOST, halo=halo,
                            proc_grid=grid)
    assert ctx.local_dims == L
    outs = {}
    for prec, recon in ((8, 18), (4, 12), (2, 12)):
        ctx.gauge_load(U, 0.12, 1.0, prec=prec, recon=recon, t_boundary=-1)
        fi, fo, fx = ctx.new_field(prec), ctx.new_field(prec), ctx.new_field(prec)
        for p in (0, 1):
            ctx.spinor_load(fi, prec, 1 - p, psi)
            ctx.spinor_load(fx, prec, p, xin)
            for dag in (0, 1):
                for kind in (0, 1, 2):
                    ctx.dslash(fo, fi, prec, p, dagger=dag, kind=kind, x=fx, a=-0.3)
                    outs[(prec, p, dag, kind)] = ctx.spinor_store(fo, prec, p)
        fa, fb = ctx.new_field(prec), ctx.new_field(prec)
        ctx.spinor_load(fa, prec, 0, psi)
        ctx.mdagm(fb, fa, prec)
        outs[(prec, "mdagm")] = ctx.spinor_store(fb, prec, 0)
        outs[(prec, "norm2")] = ctx.norm2(fb, prec)
    # solver across ranks (global reductions through the transport)
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12, t_boundary=-1)
    b = box(qgen.point_source(dims, 0, 1))
    x, st = ctx.solve(b, tol=1e-10, delta=0.1, maxiter=2000, prec=8, prec_sloppy=4)
    outs["solve_x"] = x
    outs["solve_stats"] = st
    # batched solve of three sources (multi-RHS halo: one exchange per direction carries every
    # right-hand side's face) against three independent solves: bitwise the same iterates
    srcs = [box(qgen.point_source(dims, sp, co)) for sp, co in ((0, 1), (1, 0), (0, 2))]
    xs, sts = ctx.solve_multi(srcs, tol=1e-10, delta=0.1, maxiter=2000, prec=8, prec_sloppy=4)
    same = True
    for j, bj in enumerate(srcs):
        xj, stj = ctx.solve(bj, tol=1e-10, delta=0.1, maxiter=2000, prec=8, prec_sloppy=4)
        same &= bool(np.array_equal(xj, xs[j])) and stj["iters"] == sts[j]["iters"]
    outs["batched_same"] = same
    outs["origin"] = o
    ctx.close()

    # gather slabs to rank 0
    gathered = [None] * n
    dist.gather_object(outs, gathered if rank == 0 else None, dst=0)
    def assemble(key):
        """global array from the ranks' boxes"""
        first = gathered[0][key]
        out = np.empty((dims[3], dims[2], dims[1], dims[0]) + first.shape[4:], dtype=first.dtype)
        for g in gathered:
            og = g["origin"]
            out[og[3]:og[3] + L[3], og[2]:og[2] + L[2], og[1]:og[1] + L[1], og[0]:og[0] + L[0]] = g[key]
        return out

    if rank == 0:
        ref = qudax.Context(dims, device=device)
        Ug = qgen.gauge(dims, 1301, eps=-1.0)
        pg, xg = qgen.spinor(dims, 1302), qgen.spinor(dims, 1303)
        for prec, recon in ((8, 18), (4, 12), (2, 12)):
            ref.gauge_load(Ug, 0.12, 1.0, prec=prec, recon=recon, t_boundary=-1)
            fi, fo, fx = ref.new_field(prec), ref.new_field(prec), ref.new_field(prec)
            for p in (0, 1):
                ref.spinor_load(fi, prec, 1 - p, pg)
                ref.spinor_load(fx, prec, p, xg)
                for dag in (0, 1):
                    for kind in (0, 1, 2):
                        ref.dslash(fo, fi, prec, p, dagger=dag, kind=kind, x=fx, a=-0.3)
                        want = ref.spinor_store(fo, prec, p)
                        got = assemble((prec, p, dag, kind))
                        same = bool(np.array_equal(got, want))
                        result["checks"][f"dslash p{prec} par{p} dag{dag} kind{kind}"] = same
                        result["ok"] &= same
            fa, fb = ref.new_field(prec), ref.new_field(prec)
            ref.spinor_load(fa, prec, 0, pg)
            ref.mdagm(fb, fa, prec)
            got = assemble((prec, "mdagm"))
            same = bool(np.array_equal(got, ref.spinor_store(fb, prec, 0)))
            result["checks"][f"mdagm p{prec}"] = same
            result["ok"] &= same
            # global norm equals the single-context norm up to summation order
            n_ref = ref.norm2(fb, prec)
            close = abs(gathered[0][(prec, "norm2")] - n_ref) <= 1e-12 * n_ref
            result["checks"][f"norm2 p{prec}"] = close
            result["ok"] &= close
        ref.close()
        # solver: oracle true residual of the gathered solution
        import oracle
        wc = oracle.WilsonClover(Ug, 0.124, 1.0, -1.0)
        xg_ = assemble("solve_x")
        bg = qgen.point_source(dims, 0, 1)
        res = float(np.linalg.norm(wc.M(xg_) - bg) / np.linalg.norm(bg))
        result["solve"] = {"oracle_true_res": res, "stats": gathered[0]["solve_stats"]}
        okres = res <= 1e-10 * 1.001 and abs(res - gathered[0]["solve_stats"]["true_res"]) <= 1e-9
        result["checks"]["solve"] = okres
        result["ok"] &= okres
        bsame = all(g["batched_same"] for g in gathered)
        result["checks"]["batched == independent (bitwise)"] = bsame
        result["ok"] &= bsame
        json.dump(result, open(args.out, "w"), indent=1)
    dist.barrier()
    dist.destroy_process_group()


if __name__ == "__main__":
    main()
