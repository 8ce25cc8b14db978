"""Multi-RHS Dslash / Mhat: one launch for several right-hand sides must be
bitwise equal to the single-RHS kernels (same per-site code), and within tolerance of the oracle."""
import numpy as np
import pytest

import oracle
import qgen
from paper_1011_0024_b200 import qudax
from conftest import TOL, rel_l2

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("prec,recon", [(4, 12), (4, 18), (4, 8), (2, 12), (2, 18), (2, 8), (8, 18)])
@pytest.mark.parametrize("nrhs", [2, 3, 8])
def test_multi_rhs_bitwise_and_oracle(torch_cuda, prec, recon, nrhs):
    dims = (8, 4, 6, 8)
    U = qgen.gauge(dims, 1401)
    psis = [qgen.spinor(dims, 1500 + k) for k in range(nrhs)]
    ctx = qudax.Context(dims)
    ctx.gauge_load(U, 0.12, 1.0, prec=prec, recon=recon)
    ins = [ctx.new_field(prec) for _ in range(nrhs)]
    xs = [ctx.new_field(prec) for _ in range(nrhs)]
    for k in range(nrhs):
        ctx.spinor_load(ins[k], prec, 1, psis[k])
        ctx.spinor_load(xs[k], prec, 0, psis[(k + 1) % nrhs])
    # every kind (incl. xpay with a = 0 and the symmetric-Schur inverse-xpay), both daggers; the
    # fp32 / half launches run two right-hand sides per thread (dslash_mr.cuh), odd counts
    # repeat the last one
    for dagger in (False, True):
        for kind, a in ((0, -0.3), (1, -0.3), (2, -0.3), (2, 0.0), (3, -0.3)):
            outs = [ctx.new_field(prec) for _ in range(nrhs)]
            ctx.dslash_multi(outs, ins, prec, 0, dagger=dagger, kind=kind, xs=xs, a=a)
            for k in range(nrhs):
                single = ctx.new_field(prec)
                ctx.dslash(single, ins[k], prec, 0, dagger=dagger, kind=kind, x=xs[k], a=a)
                ctx.sync()
                assert bool((single == outs[k]).all()), (dagger, kind, a, k)
    # Mhat on nrhs even fields vs the oracle
    wc = oracle.WilsonClover(U, 0.12, 1.0, -1.0)
    ev = [ctx.new_field(prec) for _ in range(nrhs)]
    for k in range(nrhs):
        ctx.spinor_load(ev[k], prec, 0, psis[k])
    outs = [ctx.new_field(prec) for _ in range(nrhs)]
    ctx.matpc_multi(outs, ev, prec)
    for k in range(nrhs):
        got = oracle.restrict(ctx.spinor_store(outs[k], prec, 0), 0)
        assert rel_l2(got, wc.matpc(oracle.restrict(psis[k], 0))) <= TOL[prec]
    ctx.close()


def test_multirhs_fused_reductions_match_single(torch_cuda):
    """Per-RHS fused reductions of the multi-RHS Mhat (through the batched solver's scalars):
    covered bitwise by test_solver.test_batched_solve_equals_independent_solves; here the
    error paths: the symmetric Schur form has no multi-RHS Mhat."""
    import qgen
    from paper_1011_0024_b200 import qudax
    dims = (8, 4, 4, 8)
    ctx = qudax.Context(dims)
    ctx.gauge_load(qgen.gauge(dims, 7), 0.12, 1.0, prec=4, recon=12)
    with pytest.raises(qudax.QudaxError):
        ctx.solve_multi([qgen.point_source(dims, 0, 0)], use_schur=2)
    ctx.close()


@pytest.mark.parametrize("prec,recon", [(4, 12), (2, 12), (8, 18)])
@pytest.mark.parametrize("overlap", [True, False])
def test_multi_rhs_halo_loopback_bitwise(torch_cuda, prec, recon, overlap):
    """The multi-RHS T halo (one exchange per direction carries every right-hand side's face;
    interior / boundary ranges of the multi-RHS kernel) through NCCL loopback at N = 1: every
    kind and dagger bitwise equal to the unpartitioned multi-RHS launch (the exchange moves bits
    only and the per-site code is the same)."""
    dims = (8, 4, 6, 8)
    nrhs = 3
    U = qgen.gauge(dims, 1411)
    psis = [qgen.spinor(dims, 1600 + k) for k in range(nrhs)]
    outs = {}
    for comm in (qudax.COMM_NONE, qudax.COMM_NCCL):
        ctx = qudax.Context(dims, comm=comm, overlap=overlap, nccl_id=qudax.nccl_unique_id() if comm else None)
        ctx.gauge_load(U, 0.12, 1.0, prec=prec, recon=recon)
        ins = [ctx.new_field(prec) for _ in range(nrhs)]
        xs = [ctx.new_field(prec) for _ in range(nrhs)]
        for k in range(nrhs):
            ctx.spinor_load(ins[k], prec, 1, psis[k])
            ctx.spinor_load(xs[k], prec, 0, psis[(k + 1) % nrhs])
        res = []
        for dagger in (False, True):
            for kind in (0, 1, 2, 3):
                o = [ctx.new_field(prec) for _ in range(nrhs)]
                ctx.dslash_multi(o, ins, prec, 0, dagger=dagger, kind=kind, xs=xs, a=-0.3)
                ctx.sync()
                res += [f.cpu().numpy().copy() for f in o]
        ev = [ctx.new_field(prec) for _ in range(nrhs)]
        for k in range(nrhs):
            ctx.spinor_load(ev[k], prec, 0, psis[k])
        o = [ctx.new_field(prec) for _ in range(nrhs)]
        ctx.matpc_multi(o, ev, prec)
        ctx.sync()
        res += [f.cpu().numpy().copy() for f in o]
        outs[comm] = res
        ctx.close()
    for a, b in zip(outs[qudax.COMM_NONE], outs[qudax.COMM_NCCL]):
        assert np.array_equal(a, b)


def test_batched_solve_loopback_multi_rhs_halo(torch_cuda):
    """Batched solve through the multi-RHS halo + per-RHS ncclAllReduce (NCCL loopback, no
    overlap so the reductions keep the unsplit CTA grouping): bitwise the unpartitioned batched
    solve, and each system bitwise its own single solve."""
    dims = (8, 8, 8, 16)
    U = qgen.gauge(dims, 1003, eps=0.1)
    srcs = [qgen.point_source(dims, s, c) for s, c in ((0, 0), (1, 2), (0, 1))]
    res = {}
    for comm in (qudax.COMM_NONE, qudax.COMM_NCCL):
        ctx = qudax.Context(dims, comm=comm, overlap=False, nccl_id=qudax.nccl_unique_id() if comm else None)
        ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        xs, sts = ctx.solve_multi(srcs, tol=1e-10, delta=1e-2, maxiter=2000, prec=8, prec_sloppy=4)
        res[comm] = (xs, [s["iters"] for s in sts])
        if comm == qudax.COMM_NCCL:
            for j, b in enumerate(srcs):
                x1, st1 = ctx.solve(b, tol=1e-10, delta=1e-2, maxiter=2000, prec=8, prec_sloppy=4)
                assert st1["iters"] == sts[j]["iters"]
                assert np.array_equal(x1, xs[j])
        ctx.close()
    assert res[qudax.COMM_NONE][1] == res[qudax.COMM_NCCL][1]
    for a, b in zip(res[qudax.COMM_NONE][0], res[qudax.COMM_NCCL][0]):
        assert np.array_equal(a, b)
