"""Split (halo) path at N=1: faces go pack -> NCCL send/recv to self -> ghost buffers ->
interior + boundary kernels, or (QUDAX_HALO_P2P) the pack kernel stores them straight into the
ghost buffers and raises the sequence flags the boundary kernel acquires.  Must be BITWISE
equal to the unsplit single-kernel path (the exchange moves bits only), overlapped or not, for
every precision and dagger."""
import numpy as np
import pytest

import qgen
from paper_1011_0024_b200 import qudax

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("prec", [8, 4, 2])
@pytest.mark.parametrize("overlap", [True, False])
@pytest.mark.parametrize("halo", ["nccl", "p2p"])
def test_loopback_bitwise(torch_cuda, prec, overlap, halo):
    dims = (8, 4, 6, 8)
    U = qgen.gauge(dims, 1201)
    psi = qgen.spinor(dims, 1202)
    x = qgen.spinor(dims, 1203)
    ref = qudax.Context(dims)
    if halo == "nccl":
        loop = qudax.Context(dims, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), overlap=overlap)
    else:
        loop = qudax.Context(dims, overlap=overlap, halo=qudax.HALO_P2P)
    for c in (ref, loop):
        c.gauge_load(U, 0.12, 1.0, prec=prec, recon=12)
    outs = {}
    for name, c in (("ref", ref), ("loop", loop)):
        fi, fo, fx = c.new_field(prec), c.new_field(prec), c.new_field(prec)
        res = []
        for p in (0, 1):
            c.spinor_load(fi, prec, 1 - p, psi)
            c.spinor_load(fx, prec, p, x)
            for dagger in (False, True):
                for kind in (0, 1, 2):
                    c.dslash(fo, fi, prec, p, dagger=dagger, kind=kind, x=fx, a=-0.2)
                    c.sync()
                    res.append(fo.cpu().numpy().copy())
        # back-to-back operators: the second exchange must not race the first boundary kernel
        fa, fb, fc = c.new_field(prec), c.new_field(prec), c.new_field(prec)
        c.spinor_load(fa, prec, 0, psi)
        c.matpc(fb, fa, prec)
        c.matpc(fc, fb, prec, dagger=True)
        c.mdagm(fb, fc, prec)
        c.sync()
        res.append(fb.cpu().numpy().copy())
        outs[name] = res
    for a, b in zip(outs["ref"], outs["loop"]):
        assert np.array_equal(a, b)
    ref.close()
    loop.close()


@pytest.mark.parametrize("mask", [0b0100, 0b0110, 0b0001, 0b1111])
@pytest.mark.parametrize("prec", [8, 4, 2])
def test_loopback_split_dims_bitwise(torch_cuda, prec, mask):
    """Multi-dimensional split path at N=1: every dimension in `mask` sends
    its faces to itself through NCCL (X/Y/Z faces spin-projected by the pack kernel in the
    arithmetic precision), interior box + boundary-list kernels; bitwise = unsplit."""
    dims = (8, 4, 6, 8)
    U = qgen.gauge(dims, 1221)
    psi = qgen.spinor(dims, 1222)
    x = qgen.spinor(dims, 1223)
    ref = qudax.Context(dims)
    loop = qudax.Context(dims, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), split_mask=mask)
    assert loop.partition["split_mask"] == mask
    outs = {}
    for name, c in (("ref", ref), ("loop", loop)):
        c.gauge_load(U, 0.12, 1.0, prec=prec, recon=12)
        fi, fo, fx = c.new_field(prec), c.new_field(prec), c.new_field(prec)
        res = []
        for p in (0, 1):
            c.spinor_load(fi, prec, 1 - p, psi)
            c.spinor_load(fx, prec, p, x)
            for dagger in (False, True):
                for kind in (0, 1, 2, 3):
                    c.dslash(fo, fi, prec, p, dagger=dagger, kind=kind, x=fx, a=-0.2)
                    c.sync()
                    res.append(fo.cpu().numpy().copy())
        fa, fb, fc = c.new_field(prec), c.new_field(prec), c.new_field(prec)
        c.spinor_load(fa, prec, 0, psi)
        c.matpc(fb, fa, prec)
        c.matpc(fc, fb, prec, dagger=True)
        c.mdagm(fb, fc, prec)
        c.sync()
        res.append(fb.cpu().numpy().copy())
        outs[name] = res
    for k, (a, b) in enumerate(zip(outs["ref"], outs["loop"])):
        assert np.array_equal(a, b), k
    ref.close()
    loop.close()


@pytest.mark.parametrize("mask", [0b0100, 0b1100, 0b0001, 0b1111])
@pytest.mark.parametrize("prec", [8, 4, 2])
@pytest.mark.parametrize("overlap", [True, False])
def test_p2p_split_dims_bitwise(torch_cuda, prec, mask, overlap):
    """Kernel-initiated halo of a multi-dimensional split (SURVEY 8(f) item 1 for X / Y / Z
    faces), loopback at N = 1: ONE pack kernel stores every split dimension's faces into the
    (own) ghost buffers and raises the per-dimension flags; ONE Dslash launch runs the interior
    box first and the boundary list in the CTAs that acquire the flags (overlap), or waits in
    every CTA (no overlap).  Bitwise = unsplit for every precision, kind, parity and dagger."""
    dims = (8, 4, 6, 8)
    U = qgen.gauge(dims, 1241)
    psi = qgen.spinor(dims, 1242)
    x = qgen.spinor(dims, 1243)
    ref = qudax.Context(dims)
    loop = qudax.Context(dims, halo=qudax.HALO_P2P, split_mask=mask, overlap=overlap)
    assert loop.partition["split_mask"] == mask
    outs = {}
    for name, c in (("ref", ref), ("loop", loop)):
        c.gauge_load(U, 0.12, 1.0, prec=prec, recon=12)
        fi, fo, fx = c.new_field(prec), c.new_field(prec), c.new_field(prec)
        res = []
        for p in (0, 1):
            c.spinor_load(fi, prec, 1 - p, psi)
            c.spinor_load(fx, prec, p, x)
            for dagger in (False, True):
                for kind in (0, 1, 2, 3):
                    c.dslash(fo, fi, prec, p, dagger=dagger, kind=kind, x=fx, a=-0.2)
                    c.sync()
                    res.append(fo.cpu().numpy().copy())
        fa, fb, fc = c.new_field(prec), c.new_field(prec), c.new_field(prec)
        c.spinor_load(fa, prec, 0, psi)
        c.matpc(fb, fa, prec)
        c.matpc(fc, fb, prec, dagger=True)
        c.mdagm(fb, fc, prec)
        c.sync()
        res.append(fb.cpu().numpy().copy())
        outs[name] = res
    for k, (a, b) in enumerate(zip(outs["ref"], outs["loop"])):
        assert np.array_equal(a, b), k
    ref.close()
    loop.close()


def test_p2p_split_dims_solve(torch_cuda):
    """Mixed-precision solve with Y, Z and T split through the kernel-initiated halo and the
    kernel-side allreduce (loopback, graph replay): the unsplit solve's iterations and solution
    (fp32 sloppy: the fused reductions' fp64 sums of fp32 site partials are exact, so the
    different CTA grouping of the tail launch does not change them)."""
    dims = (8, 4, 4, 16)
    U = qgen.gauge(dims, 1251, eps=0.1)
    b = qgen.point_source(dims, 0, 2)
    res = {}
    for name, kw in (("ref", {}), ("p2p", {"halo": qudax.HALO_P2P, "split_mask": 0b1110})):
        c = qudax.Context(dims, **kw)
        c.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        x, st = c.solve(b, tol=1e-12, delta=0.1, maxiter=1000, prec=8, prec_sloppy=4)
        res[name] = (x, st)
        c.close()
    assert res["ref"][1]["iters"] == res["p2p"][1]["iters"]
    rel = np.linalg.norm(res["ref"][0] - res["p2p"][0]) / np.linalg.norm(res["ref"][0])
    assert rel < 1e-12


def test_p2p_loopback_solve(torch_cuda):
    """Mixed-precision solve through the kernel-initiated halo (graph replay included): same
    iterations and residual history as the unsplit context (bitwise operators)."""
    dims = (8, 4, 4, 16)
    U = qgen.gauge(dims, 1211, eps=0.1)
    b = qgen.point_source(dims, 0, 0)
    res = {}
    for name, kw in (("ref", {}), ("p2p", {"halo": qudax.HALO_P2P})):
        c = qudax.Context(dims, **kw)
        c.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        x, st = c.solve(b, tol=1e-12, delta=0.1, maxiter=1000, prec=8, prec_sloppy=4)
        res[name] = (x, st)
        c.close()
    assert res["ref"][1]["iters"] == res["p2p"][1]["iters"]
    assert np.array_equal(res["ref"][0], res["p2p"][0])


def test_loopback_split_dims_solve(torch_cuda):
    """Mixed-precision solve with Y, Z and T split in loopback (NCCL to self, CUDA-graph
    replay of the iteration included): bitwise the unsplit solve."""
    dims = (8, 4, 4, 16)
    U = qgen.gauge(dims, 1231, eps=0.1)
    b = qgen.point_source(dims, 1, 2)
    res = {}
    for name, kw in (("ref", {}), ("split", {"comm": qudax.COMM_NCCL, "nccl_id": qudax.nccl_unique_id(),
                                               "split_mask": 0b1110})):
        c = qudax.Context(dims, **kw)
        c.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
        x, st = c.solve(b, tol=1e-12, delta=0.1, maxiter=1000, prec=8, prec_sloppy=4)
        res[name] = (x, st)
        c.close()
    assert res["ref"][1]["iters"] == res["split"][1]["iters"]
    assert np.array_equal(res["ref"][0], res["split"][0])


def test_halo_timeline_shows_overlap(torch_cuda):
    """The NCCL path's pack + exchange run on the comm stream while the interior kernel runs on
    the compute stream: events on both streams (qudax_halo_timeline) must show the
    comm-stream work starting before the interior kernel ends, and the boundary kernel starting
    only after the exchange ended."""
    dims = (16, 16, 16, 32)
    ctx = qudax.Context(dims, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), overlap=True)
    ctx.gauge_load(qgen.gauge(dims, 1261), 0.12, 1.0, prec=4, recon=12)
    fi, fo = ctx.new_field(4), ctx.new_field(4)
    ctx.spinor_load(fi, 4, 0, qgen.spinor(dims, 1262))
    ctx.matpc(fo, fi, 4)
    ctx.halo_timeline(True)
    ctx.matpc(fo, fi, 4)
    m = ctx.halo_timeline(False, read=True)
    ctx.close()
    order = ["pack_start", "exchange_start", "exchange_end"]
    assert all(m[a] <= m[b] for a, b in zip(order, order[1:])), m
    assert m["interior_start"] <= m["interior_end"] <= m["boundary_start"] <= m["boundary_end"], m
    assert m["pack_start"] < m["interior_end"], m        # the halo work began while the interior ran
    assert m["boundary_start"] >= m["exchange_end"], m   # the boundary waited for the ghosts
