"""GPU Dslash / Mhat parity against the fp64 oracle (BASELINE configs 1 and 2).

Every case runs through the C-ABI (paper_1011_0024_b200.qudax -> libqudax.so) on seeded
inputs from qgen, and compares with oracle/ element by element (relative L2 over the output
parity's sites) at the north_star tolerances: fp64 1e-12, fp32 1e-5, half 5e-3.
"""
import numpy as np
import pytest

import oracle
import qgen
from paper_1011_0024_b200 import qudax
from conftest import TOL, rel_l2

pytestmark = pytest.mark.gpu

KAPPA, CSW = 0.12, 1.0


class Case:
    def __init__(self, dims, gseed, sseed, eps=-1.0, kappa=KAPPA, csw=CSW, t_bc=-1):
        self.dims = dims
        self.U = qgen.gauge(dims, gseed, eps=eps)
        self.psi = qgen.spinor(dims, sseed)
        self.x = qgen.spinor(dims, sseed + 1)
        self.kappa, self.csw, self.t_bc = kappa, csw, t_bc
        self.wc = oracle.WilsonClover(self.U, kappa, csw, t_bc)

    def expect(self, p, dagger, kind, a=0.0):
        d = self.wc.Dpq(self.psi, p, dagger)
        if kind == qudax.HOP:
            return d
        if kind == qudax.CLOVER_INV:
            return self.wc.Tinv_pp(d, p)
        return self.wc.Tpp(self.x, p) + a * d


_cases = {}


def get_case(name):
    if name not in _cases:
        if name == "4^4":
            _cases[name] = Case((4, 4, 4, 4), 1001, 2001)
        elif name == "8x4x6x8":
            _cases[name] = Case((8, 4, 6, 8), 1011, 2011)
        elif name == "16^3x32":
            _cases[name] = Case((16, 16, 16, 32), 1002, 2002)
        elif name == "8x4x6x8 periodic":
            _cases[name] = Case((8, 4, 6, 8), 1011, 2011, t_bc=+1)
        elif name == "16^3x32 periodic":
            _cases[name] = Case((16, 16, 16, 32), 1002, 2002, t_bc=+1)
    return _cases[name]


def make_ctx(case, prec, recon, comm=qudax.COMM_NONE, nccl_id=None):
    ctx = qudax.Context(case.dims, comm=comm, nccl_id=nccl_id)
    ctx.gauge_load(case.U, case.kappa, case.csw, prec=prec, recon=recon, t_boundary=case.t_bc)
    return ctx


def run_dslash(ctx, case, prec, p, dagger, kind, a=0.0):
    fin, fout, fx = ctx.new_field(prec), ctx.new_field(prec), ctx.new_field(prec)
    ctx.spinor_load(fin, prec, 1 - p, case.psi)
    ctx.spinor_load(fx, prec, p, case.x)
    ctx.dslash(fout, fin, prec, p, dagger=dagger, kind=kind, x=fx, a=a)
    return oracle.restrict(ctx.spinor_store(fout, prec, p), p)


@pytest.mark.parametrize("prec", [8, 4, 2])
@pytest.mark.parametrize("recon", [18, 12, 8])
def test_dslash_matrix_16x32(torch_cuda, prec, recon):
    """BJ config 2: 16^3x32, Haar gauge, {fp64,fp32,half} x {18,12,8} x parity x dagger x kind."""
    case = get_case("16^3x32")
    ctx = make_ctx(case, prec, recon)
    worst = 0.0
    for p in (0, 1):
        for dagger in (False, True):
            for kind in (qudax.HOP, qudax.CLOVER_INV, qudax.CLOVER_XPAY):
                a = -0.37
                got = run_dslash(ctx, case, prec, p, dagger, kind, a)
                e = rel_l2(got, case.expect(p, dagger, kind, a))
                worst = max(worst, e)
                assert e <= TOL[prec], (prec, recon, p, dagger, kind, e)
    print(f"prec={prec} recon={recon} worst rel-L2 {worst:.3e}")
    ctx.close()


@pytest.mark.parametrize("name", ["4^4", "8x4x6x8"])
@pytest.mark.parametrize("prec", [8, 4, 2])
def test_dslash_small_lattices(torch_cuda, name, prec):
    """BJ config 1 (4^4) and a rectangular lattice; plain Wilson (csw = 0) and clover."""
    case = get_case(name)
    for recon in (18, 12):
        ctx = make_ctx(case, prec, recon)
        for p in (0, 1):
            for dagger in (False, True):
                for kind in (0, 1, 2):
                    got = run_dslash(ctx, case, prec, p, dagger, kind, 0.5)
                    assert rel_l2(got, case.expect(p, dagger, kind, 0.5)) <= TOL[prec]
        ctx.close()


@pytest.mark.parametrize("prec", [8, 4, 2])
@pytest.mark.parametrize("recon", [18, 12, 8])
def test_dslash_periodic_t(torch_cuda, prec, recon):
    """t_boundary = +1 (periodic in T; P:381-383 and P:625-628 leave the boundary constants to
    the caller, reading Q5): every precision, reconstruct, parity, dagger and kind at 16^3x32,
    Mhat and Mhat^dag at 8x4x6x8.  With recon 12 the third row is rebuilt BEFORE the sign, so an
    in-storage sign flip would fail here and in the antiperiodic matrix alike."""
    case = get_case("16^3x32 periodic")
    ctx = make_ctx(case, prec, recon)
    for p in (0, 1):
        for dagger in (False, True):
            for kind in (qudax.HOP, qudax.CLOVER_INV, qudax.CLOVER_XPAY):
                got = run_dslash(ctx, case, prec, p, dagger, kind, -0.37)
                e = rel_l2(got, case.expect(p, dagger, kind, -0.37))
                assert e <= TOL[prec], (prec, recon, p, dagger, kind, e)
    ctx.close()
    small = get_case("8x4x6x8 periodic")
    ctx = make_ctx(small, prec, recon)
    psi_e = oracle.restrict(small.psi, 0)
    fin, fout = ctx.new_field(prec), ctx.new_field(prec)
    ctx.spinor_load(fin, prec, 0, small.psi)
    for dagger in (False, True):
        ctx.matpc(fout, fin, prec, dagger)
        got = oracle.restrict(ctx.spinor_store(fout, prec, 0), 0)
        assert rel_l2(got, small.wc.matpc(psi_e, dagger)) <= TOL[prec], dagger
    # the periodic and antiperiodic operators must differ (the sign is not silently dropped)
    anti = oracle.WilsonClover(small.U, small.kappa, small.csw, -1).matpc(psi_e)
    assert rel_l2(got, anti) > 0.05  # measured 0.11 in fp64 on this lattice
    ctx.close()


def test_wilson_csw0_4x4(torch_cuda):
    case = Case((4, 4, 4, 4), 1001, 2001, kappa=0.12, csw=0.0)
    ctx = make_ctx(case, 8, 18)
    for kind in (1, 2):
        got = run_dslash(ctx, case, 8, 0, False, kind, -0.1)
        assert rel_l2(got, case.expect(0, False, kind, -0.1)) <= 1e-12
    ctx.close()


@pytest.mark.parametrize("prec,recon", [(8, 18), (4, 12), (2, 12), (4, 8)])
def test_matpc_and_mdagm(torch_cuda, prec, recon):
    case = get_case("8x4x6x8")
    ctx = make_ctx(case, prec, recon)
    psi_e = oracle.restrict(case.psi, 0)
    fin, fout = ctx.new_field(prec), ctx.new_field(prec)
    ctx.spinor_load(fin, prec, 0, case.psi)
    for dagger in (False, True):
        ctx.matpc(fout, fin, prec, dagger)
        got = oracle.restrict(ctx.spinor_store(fout, prec, 0), 0)
        assert rel_l2(got, case.wc.matpc(psi_e, dagger)) <= TOL[prec]
    ctx.mdagm(fout, fin, prec)
    got = oracle.restrict(ctx.spinor_store(fout, prec, 0), 0)
    assert rel_l2(got, case.wc.mdagm(psi_e)) <= TOL[prec]
    ctx.close()


@pytest.mark.parametrize("prec,recon", [(8, 18), (4, 12), (2, 12)])
def test_matpc_sym_and_kernel_kind3(torch_cuda, prec, recon):
    """Symmetric Schur form and its kernel CLOVER_INV_XPAY
    (out = x + a T^{-1} D in) against the oracle, both parities and daggers."""
    case = get_case("8x4x6x8")
    ctx = make_ctx(case, prec, recon)
    for p in (0, 1):
        for dagger in (False, True):
            got = run_dslash(ctx, case, prec, p, dagger, qudax.CLOVER_INV_XPAY, -0.29)
            want = oracle.restrict(case.x, p) - 0.29 * case.wc.Tinv_pp(case.wc.Dpq(case.psi, p, dagger), p)
            assert rel_l2(got, want) <= TOL[prec], (p, dagger)
    psi_e = oracle.restrict(case.psi, 0)
    fin, fout = ctx.new_field(prec), ctx.new_field(prec)
    ctx.spinor_load(fin, prec, 0, case.psi)
    for dagger in (False, True):
        ctx.matpc_sym(fout, fin, prec, dagger)
        got = oracle.restrict(ctx.spinor_store(fout, prec, 0), 0)
        assert rel_l2(got, case.wc.matpc_sym(psi_e, dagger)) <= TOL[prec], dagger
    ctx.close()


def test_free_field_matpc_closed_form(torch_cuda):
    """Analytic check with no oracle: unit gauge (T = 1), plane wave on even sites."""
    dims = (8, 4, 4, 8)
    kappa = 0.12
    X, Y, Z, T = dims
    p = [2 * np.pi / X, 2 * np.pi * 2 / Y, 0.0, 3 * np.pi / T]
    rng = np.random.default_rng(5)
    u = rng.normal(size=(4, 3)) + 1j * rng.normal(size=(4, 3))
    t, z, y, x = np.meshgrid(np.arange(T), np.arange(Z), np.arange(Y), np.arange(X), indexing="ij")
    pw = np.exp(1j * (p[0] * x + p[1] * y + p[2] * z + p[3] * t))[..., None, None] * u
    # NR-independent closed form in the DR basis, gamma matrices from SURVEY App. A
    i = 1j
    G = [np.array([[0, 0, 0, i], [0, 0, i, 0], [0, -i, 0, 0], [-i, 0, 0, 0]]),
         np.array([[0, 0, 0, -1], [0, 0, 1, 0], [0, 1, 0, 0], [-1, 0, 0, 0]], dtype=complex),
         np.array([[0, 0, i, 0], [0, 0, 0, -i], [-i, 0, 0, 0], [0, i, 0, 0]]),
         np.array([[0, 0, 1, 0], [0, 0, 0, 1], [1, 0, 0, 0], [0, 1, 0, 0]], dtype=complex)]
    Dt = sum(2 * np.cos(p[m]) * np.eye(4) - 2j * np.sin(p[m]) * G[m] for m in range(4))
    expect = oracle.restrict(np.einsum("st,...tc->...sc", np.eye(4) - kappa ** 2 * Dt @ Dt, pw), 0)
    for prec, tol in ((8, 1e-13), (4, 1e-5)):
        ctx = qudax.Context(dims)
        ctx.gauge_load(qgen.unit_gauge(dims), kappa, 1.0, prec=prec, recon=12, t_boundary=-1)
        fin, fout = ctx.new_field(prec), ctx.new_field(prec)
        ctx.spinor_load(fin, prec, 0, pw)
        ctx.matpc(fout, fin, prec)
        got = oracle.restrict(ctx.spinor_store(fout, prec, 0), 0)
        assert np.abs(got - expect).max() / np.abs(expect).max() < tol
        ctx.close()


def test_recon8_rejects_unit_gauge(torch_cuda):
    dims = (4, 4, 4, 4)
    ctx = qudax.Context(dims)
    with pytest.raises(qudax.QudaxError) as ei:
        ctx.gauge_load(qgen.unit_gauge(dims), 0.12, 1.0, prec=4, recon=8)
    assert ei.value.status == 5
    ctx.close()


@pytest.mark.parametrize("prec", [8, 4, 2])
def test_layout_roundtrip(torch_cuda, prec):
    dims = (8, 4, 6, 8)
    psi = qgen.spinor(dims, 9)
    ctx = qudax.Context(dims)
    out = np.zeros_like(psi)
    for parity in (0, 1):
        f = ctx.new_field(prec)
        ctx.spinor_load(f, prec, parity, psi)
        ctx.spinor_store(f, prec, parity, out)
    err = np.abs(out - psi).max()
    if prec == 8:
        assert err < 1e-15 * np.abs(psi).max() * 4
    elif prec == 4:
        assert rel_l2(out, psi) < 1e-7
    else:
        # half: per-site norm = max |real|, |v - q(v)| <= norm / 65534 per real (reading Q7);
        # the basis rotation mixes 2 components per real on the way out
        nrm = np.abs(np.stack([psi.real, psi.imag], -1)).reshape(psi.shape[:4] + (-1,)).max(-1)
        bound = 2 * (nrm / 65534.0)[..., None, None] * np.sqrt(2) * 1.01 + 1e-7
        assert np.all(np.abs(out.real - psi.real) <= bound) and np.all(np.abs(out.imag - psi.imag) <= bound)
    ctx.close()


def test_reductions_match_numpy(torch_cuda):
    dims = (8, 4, 6, 8)
    a, b = qgen.spinor(dims, 11), qgen.spinor(dims, 12)
    ctx = qudax.Context(dims)
    fa, fb = ctx.new_field(8), ctx.new_field(8)
    ctx.spinor_load(fa, 8, 0, a)
    ctx.spinor_load(fb, 8, 0, b)
    ae, be = oracle.restrict(a, 0), oracle.restrict(b, 0)
    assert abs(ctx.norm2(fa, 8) - np.vdot(ae, ae).real) < 1e-12 * np.vdot(ae, ae).real
    assert abs(ctx.cdot(fa, fb, 8) - np.vdot(ae, be)) < 1e-12 * abs(np.vdot(ae, be)) + 1e-9
    # bitwise reproducible
    assert ctx.norm2(fa, 8) == ctx.norm2(fa, 8)
    ctx.close()
