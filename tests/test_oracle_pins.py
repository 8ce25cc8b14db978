"""Pins for the fp64 CPU oracle (oracle/), checked against what the paper and the
mathematics fix — never against the oracle itself or the CUDA path.

Each test names the oracle part it pins and the mistake class it is meant to catch.
"""
import numpy as np
import pytest

import oracle
import qgen
from qtest_util import read_golden

RNG = np.random.default_rng(12345)


def _rand_spinor(dims, seed):
    return qgen.spinor(dims, seed)


# --------------------------------------------------------------------------- gammas

def test_gamma_clifford_hermitian():
    g = [oracle.gamma(mu) for mu in range(4)]
    for a in range(4):
        assert np.allclose(g[a], g[a].conj().T, atol=0)
        for b in range(4):
            assert np.allclose(g[a] @ g[b] + g[b] @ g[a], 2 * np.eye(4) * (a == b), atol=0)
    assert np.allclose(oracle.gamma5(), np.diag([1, 1, -1, -1]), atol=0)


def test_gamma4_projectors_match_eq6():
    """P^{+-4} = 1 +- gamma_4 must reproduce eq. (6) in the chiral basis, and
    the non-relativistic basis change S must diagonalise them to the printed right side."""
    sec, _ = read_golden("eq6_projectors.txt")
    g4 = oracle.gamma(3)
    assert np.allclose(np.eye(4) + g4, np.array(sec["P+4 chiral"]), atol=0)
    assert np.allclose(np.eye(4) - g4, np.array(sec["P-4 chiral"]), atol=0)
    S = np.array([[1, 0, 1, 0], [0, 1, 0, 1], [1, 0, -1, 0], [0, 1, 0, -1]]) / np.sqrt(2)
    assert np.allclose(S @ (np.eye(4) + g4) @ S.T, np.array(sec["P+4 nonrel"]), atol=1e-15)
    assert np.allclose(S @ (np.eye(4) - g4) @ S.T, np.array(sec["P-4 nonrel"]), atol=1e-15)


def test_gammas_match_appendix_a_golden():
    """gamma_1..gamma_4 and gamma_5 entry by entry against the transcription of SURVEY.md
    Appendix A (tests/golden/gamma_degrand_rossi.txt; gamma_4 also fixed by eq. (6)).
    Clifford algebra alone admits any unitary rotation of the basis; this pins the one the API
    documents (a swapped or sign-flipped gamma_mu changes which spin components a hop mixes)."""
    sec, _ = read_golden("gamma_degrand_rossi.txt")
    for mu in range(4):
        want = np.array(sec[f"g{mu + 1} re"]) + 1j * np.array(sec[f"g{mu + 1} im"])
        assert np.array_equal(oracle.gamma(mu), want), mu
    assert np.array_equal(oracle.gamma5(), np.array(sec["g5 re"]))


# --------------------------------------------------------------------------- generators

def test_generator_su3_and_slab_independence():
    dims = (4, 2, 2, 6)
    for eps in (-1.0, 0.1):
        U = qgen.gauge(dims, 77, eps=eps)
        m = U.reshape(-1, 3, 3)
        uu = np.einsum("nij,nkj->nik", m, m.conj())
        assert np.abs(uu - np.eye(3)).max() < 1e-14
        assert np.abs(np.linalg.det(m) - 1).max() < 1e-14
        # a slab of timeslices (with wrap) equals the corresponding global slices
        slab = qgen.gauge(dims, 77, eps=eps, t_begin=4, nt=4)
        assert np.array_equal(slab[:, :2], U[:, 4:6])
        assert np.array_equal(slab[:, 2:], U[:, 0:2])
    psi = qgen.spinor(dims, 5)
    assert np.array_equal(qgen.spinor(dims, 5, t_begin=3, nt=2), psi[3:5])


def test_generator_box_equals_global_slice():
    """Process-grid boxes (multi-dimensional partitioning) draw exactly their part of the one
    global field, wrapping at the lattice edge."""
    dims = (8, 4, 6, 8)
    U, S = qgen.gauge(dims, 5, eps=0.1), qgen.spinor(dims, 6)
    ts, zs, ys, xs = [6, 7, 0, 1], [3, 4, 5], [0, 1, 2, 3], [4, 5, 6, 7]
    g = qgen.gauge_box(dims, 5, (4, 0, 3, 6), (4, 4, 3, 4), eps=0.1)
    s = qgen.spinor_box(dims, 6, (4, 0, 3, 6), (4, 4, 3, 4))
    assert np.array_equal(g, U[:, ts][:, :, zs][:, :, :, ys][:, :, :, :, xs])
    assert np.array_equal(s, S[ts][:, zs][:, :, ys][:, :, :, xs])


def test_generator_haar_moments_and_weak_field():
    dims = (8, 8, 8, 8)
    U = qgen.gauge(dims, 3, eps=-1.0).reshape(-1, 3, 3)
    # Haar SU(3): E|U_ab|^2 = 1/3, E U_ab = 0, E tr U = 0
    assert abs(np.mean(np.abs(U[:, 0, 0]) ** 2) - 1 / 3) < 0.01
    assert abs(np.mean(np.abs(U[:, 2, 1]) ** 2) - 1 / 3) < 0.01
    assert abs(np.mean(np.trace(U, axis1=1, axis2=2))) < 0.02
    W = qgen.gauge(dims, 3, eps=0.1).reshape(-1, 3, 3)
    assert np.mean(np.real(np.trace(W, axis1=1, axis2=2))) > 2.8  # near identity


# --------------------------------------------------------------------------- hopping term D

@pytest.mark.parametrize("t_bc", [1.0, -1.0])
def test_dslash_gamma5_hermiticity(t_bc):
    """(i) <phi, D psi> = <D^dag phi, psi>; (ii) gamma5 D gamma5 psi = D^dag psi.
    Catches a wrong adjoint (missing conj/transposed link) or wrong dagger projectors."""
    dims = (4, 4, 2, 4)
    U = qgen.gauge(dims, 11)
    phi, psi = _rand_spinor(dims, 1), _rand_spinor(dims, 2)
    Dpsi = oracle.dslash(U, psi, t_bc)
    Ddphi = oracle.dslash(U, phi, t_bc, dagger=True)
    lhs, rhs = np.vdot(phi, Dpsi), np.vdot(Ddphi, psi)
    assert abs(lhs - rhs) / abs(lhs) < 1e-14
    g5 = oracle.gamma5()
    g5psi = np.einsum("st,...tc->...sc", g5, psi)
    lhs2 = np.einsum("st,...tc->...sc", g5, oracle.dslash(U, g5psi, t_bc))
    rhs2 = oracle.dslash(U, psi, t_bc, dagger=True)
    assert np.linalg.norm(lhs2 - rhs2) / np.linalg.norm(rhs2) < 1e-14


def _gauge_transform(U, G):
    """U^G_mu(x) = G(x) U_mu(x) G(x+mu)^dag."""
    UG = np.empty_like(U)
    for mu in range(4):
        axis = 3 - mu  # arrays are [t, z, y, x]
        Gp = np.roll(G, -1, axis=axis)
        UG[mu] = np.einsum("...ab,...bc,...dc->...ad", G, U[mu], Gp.conj())
    return UG


def test_dslash_gauge_covariance():
    """D[U^G] (G psi) = G D[U] psi.  Catches U vs U^dag mix-ups and wrong link sites."""
    dims = (4, 2, 4, 4)
    U = qgen.gauge(dims, 21)
    G = qgen.gauge_transform(dims, 22)
    psi = _rand_spinor(dims, 23)
    UG = _gauge_transform(U, G)
    Gpsi = np.einsum("...ab,...sb->...sa", G, psi)
    for dag in (False, True):
        lhs = oracle.dslash(UG, Gpsi, -1.0, dag)
        rhs = np.einsum("...ab,...sb->...sa", G, oracle.dslash(U, psi, -1.0, dag))
        assert np.linalg.norm(lhs - rhs) / np.linalg.norm(rhs) < 1e-13


def _plane_wave(dims, n, antiperiodic, u):
    X, Y, Z, T = dims
    p = [2 * np.pi * n[0] / X, 2 * np.pi * n[1] / Y, 2 * np.pi * n[2] / Z,
         ((2 * n[3] + 1) * np.pi / T) if antiperiodic else (2 * np.pi * n[3] / T)]
    t, z, y, x = np.meshgrid(np.arange(T), np.arange(Z), np.arange(Y), np.arange(X), indexing="ij")
    ph = np.exp(1j * (p[0] * x + p[1] * y + p[2] * z + p[3] * t))
    return p, ph[..., None, None] * u[None, None, None, None]


@pytest.mark.parametrize("antiperiodic", [False, True])
def test_dslash_free_field_plane_wave(antiperiodic):
    """Unit gauge, psi = e^{ip.x} u:  D psi = e^{ip.x} [sum_mu 2 cos p_mu - 2 i gamma_mu sin p_mu] u.
    Catches sign errors in 1 -+ gamma, the forward/backward assignment, and the BC."""
    dims = (6, 4, 4, 8)
    U = qgen.unit_gauge(dims)
    u = RNG.normal(size=(4, 3)) + 1j * RNG.normal(size=(4, 3))
    for n in [(1, 0, 0, 0), (0, 1, 2, 1), (2, 3, 1, 3)]:
        p, psi = _plane_wave(dims, n, antiperiodic, u)
        Dt = sum(2 * np.cos(p[m]) * np.eye(4) - 2j * np.sin(p[m]) * oracle.gamma(m) for m in range(4))
        expect = np.einsum("st,...tc->...sc", Dt, psi)
        got = oracle.dslash(U, psi, -1.0 if antiperiodic else 1.0)
        assert np.abs(got - expect).max() < 1e-13


def test_free_field_spectrum_2x4():
    """Eigenvalues of M_kappa = 1 - kappa D on the unit-gauge 2^4 lattice (antiperiodic t):
    1 - 2 kappa sum cos p -+ 2 i kappa sqrt(sum sin^2 p), each 6-fold.  The dense matrix is
    assembled column by column from the oracle's own D."""
    dims = (2, 2, 2, 2)
    kappa = 0.11
    U = qgen.unit_gauge(dims)
    N = 12 * 16
    M = np.zeros((N, N), dtype=np.complex128)
    for j in range(N):
        e = np.zeros(N, dtype=np.complex128)
        e[j] = 1
        psi = e.reshape(2, 2, 2, 2, 4, 3)
        M[:, j] = (psi - kappa * oracle.dslash(U, psi, -1.0)).reshape(-1)
    ev = np.linalg.eigvals(M)
    expect = []
    for n0 in range(2):
        for n1 in range(2):
            for n2 in range(2):
                for n3 in range(2):
                    p = [np.pi * n0, np.pi * n1, np.pi * n2, (2 * n3 + 1) * np.pi / 2]
                    a = 1 - 2 * kappa * sum(np.cos(q) for q in p)
                    b = 2 * kappa * np.sqrt(sum(np.sin(q) ** 2 for q in p))
                    expect += [a + 1j * b] * 6 + [a - 1j * b] * 6
    key = lambda z: (round(z.real, 9), round(z.imag, 9))
    assert np.allclose(sorted(ev, key=key), sorted(expect, key=key), atol=1e-12)


def test_dslash_vs_dense_bruteforce_2x4():
    """On 2^4, x+mu == x-mu: both hops land on one block — an index-bug trap.  The dense
    matrix is built entry by entry with independent index logic."""
    dims = (2, 2, 2, 2)
    U = qgen.gauge(dims, 31)
    Dd = oracle.dense_hopping(U, -1.0)
    for seed in (1, 2):
        psi = _rand_spinor(dims, seed)
        v = oracle.to_dense_vec(psi)
        assert np.abs(oracle.dslash(U, psi, -1.0).reshape(-1) - Dd @ v).max() < 1e-13
        assert np.abs(oracle.dslash(U, psi, -1.0, True).reshape(-1) - Dd.conj().T @ v).max() < 1e-13


def test_dslash_vs_dense_bruteforce_rect():
    dims = (4, 2, 2, 4)
    U = qgen.gauge(dims, 32)
    Dd = oracle.dense_hopping(U, -1.0)
    psi = _rand_spinor(dims, 3)
    assert np.abs(oracle.dslash(U, psi, -1.0).reshape(-1) - Dd @ oracle.to_dense_vec(psi)).max() < 1e-13


def test_dslash_slab_offset_matches_global():
    """A T-slab with one halo timeslice each side, placed with t_global_offset, reproduces
    the global result on its interior (the oracle's bounded-memory mode for big lattices)."""
    dims = (4, 2, 2, 8)
    U = qgen.gauge(dims, 41)
    psi = qgen.spinor(dims, 42)
    full = oracle.dslash(U, psi, -1.0)
    for t0, nt in ((0, 4), (4, 4), (2, 2)):
        Us = qgen.gauge(dims, 41, t_begin=t0 - 1, nt=nt + 2)
        ps = qgen.spinor(dims, 42, t_begin=t0 - 1, nt=nt + 2)
        out = oracle.dslash(Us, ps, -1.0, t_global_offset=t0 - 1, T_global=8)
        assert np.array_equal(out[1:-1], full[t0:t0 + nt])


# --------------------------------------------------------------------------- clover

def test_clover_abelian_closed_form():
    """Constant abelian field in the 1-2 plane, B = 2 pi n/(XY), charges q = (1,-1,0):
    T psi = (1 +- kappa csw sin(B q_a)) psi for psi = v (x) e_a with gamma1 gamma2 v = +-i v.
    Pins the 1/8, the -csw/2, leaf orientation and the sign w.r.t. the gamma convention."""
    X, Y, Z, T = 4, 4, 2, 2
    dims = (X, Y, Z, T)
    B = 2 * np.pi * 1 / (X * Y)
    q = np.array([1.0, -1.0, 0.0])
    U = qgen.unit_gauge(dims)
    for t in range(T):
        for z in range(Z):
            for y in range(Y):
                for x in range(X):
                    U[0, t, z, y, x] = np.diag(np.exp(-1j * B * y * q))
                    if y == Y - 1:
                        U[1, t, z, y, x] = np.diag(np.exp(1j * B * Y * x * q))
    kappa, csw = 0.13, 1.7
    Tm = oracle.clover(U, kappa, csw)
    g12 = oracle.gamma(0) @ oracle.gamma(1)
    w, vecs = np.linalg.eig(g12)
    for k in range(4):
        lam = w[k]
        sgn = 1 if abs(lam - 1j) < 1e-12 else -1
        assert abs(lam - sgn * 1j) < 1e-12
        for a in range(3):
            vec = np.kron(vecs[:, k], np.eye(3)[a])
            out = np.einsum("...ij,j->...i", Tm, vec)
            expect = (1 + sgn * kappa * csw * np.sin(B * q[a])) * vec
            assert np.abs(out - expect).max() < 1e-14


def test_clover_properties():
    dims = (4, 2, 2, 4)
    U = qgen.gauge(dims, 51)
    Tm = oracle.clover(U, 0.12, 1.0)
    assert np.abs(Tm - np.swapaxes(Tm.conj(), -1, -2)).max() < 1e-14  # Hermitian
    G5 = np.kron(oracle.gamma5(), np.eye(3))
    assert np.abs(G5 @ Tm - Tm @ G5).max() < 1e-14  # commutes with gamma5 -> chiral blocks
    assert np.abs(Tm[..., :6, 6:]).max() < 1e-15     # DR: exactly block diagonal
    assert np.abs(oracle.clover(U, 0.12, 0.0) - np.eye(12)).max() == 0  # csw=0: Wilson
    assert np.abs(oracle.clover(qgen.unit_gauge(dims), 0.12, 1.0) - np.eye(12)).max() < 1e-15
    assert np.abs(Tm - np.eye(12)).max() > 1e-3                     # non-trivial on Haar


def test_clover_gauge_covariance():
    dims = (4, 2, 2, 4)
    U = qgen.gauge(dims, 52)
    G = qgen.gauge_transform(dims, 53)
    Tm = oracle.clover(U, 0.12, 1.3)
    TG = oracle.clover(_gauge_transform(U, G), 0.12, 1.3)
    G12 = np.einsum("st,...ab->...satb", np.eye(4), G).reshape(G.shape[:4] + (12, 12))
    expect = G12 @ Tm @ np.swapaxes(G12.conj(), -1, -2)
    assert np.abs(TG - expect).max() < 1e-13


def test_invert12_vs_library():
    dims = (4, 2, 2, 2)
    U = qgen.gauge(dims, 54)
    Tm = oracle.clover(U, 0.125, 1.0)
    Ti = oracle.invert12(Tm)
    assert np.abs(Ti - np.linalg.inv(Tm)).max() < 1e-12


# --------------------------------------------------------------------------- even-odd and solver

def _dense_system(dims, seed, kappa, csw, t_bc=-1.0):
    U = qgen.gauge(dims, seed)
    wc = oracle.WilsonClover(U, kappa, csw, t_bc)
    Dd = oracle.dense_hopping(U, t_bc)
    V = int(np.prod(dims))
    Tblk = np.zeros((12 * V, 12 * V), dtype=np.complex128)
    Tf = wc.T.reshape(V, 12, 12)
    for s in range(V):
        Tblk[12 * s:12 * s + 12, 12 * s:12 * s + 12] = Tf[s]
    M = Tblk - kappa * Dd
    odd = oracle.parity_mask(dims).reshape(-1)
    ev_idx = np.repeat(~odd, 12)
    return wc, M, ev_idx


def test_matpc_vs_dense_schur():
    dims = (2, 2, 2, 2)
    wc, M, e = _dense_system(dims, 61, 0.124, 1.0)
    o = ~e
    Schur = M[np.ix_(e, e)] - M[np.ix_(e, o)] @ np.linalg.solve(M[np.ix_(o, o)], M[np.ix_(o, e)])
    psi = oracle.restrict(qgen.spinor(dims, 62), 0)
    v = psi.reshape(-1)[e]
    got = wc.matpc(psi).reshape(-1)
    assert np.abs(got[e] - Schur @ v).max() < 1e-13
    assert np.abs(got[o]).max() == 0
    gotd = wc.matpc(psi, dagger=True).reshape(-1)
    assert np.abs(gotd[e] - Schur.conj().T @ v).max() < 1e-13


def test_matpc_sym_vs_dense_schur():
    """Symmetric form = T_ee^{-1} (dense Schur complement), built from the dense matrix with its
    own index logic; the explicit dagger is its conjugate transpose."""
    dims = (2, 2, 2, 2)
    wc, M, e = _dense_system(dims, 66, 0.124, 1.0)
    o = ~e
    Schur = M[np.ix_(e, e)] - M[np.ix_(e, o)] @ np.linalg.solve(M[np.ix_(o, o)], M[np.ix_(o, e)])
    Sym = np.linalg.solve(M[np.ix_(e, e)], Schur)  # M_ee = T_ee on the even block
    psi = oracle.restrict(qgen.spinor(dims, 67), 0)
    v = psi.reshape(-1)[e]
    got = wc.matpc_sym(psi).reshape(-1)
    assert np.abs(got[e] - Sym @ v).max() < 1e-13
    assert np.abs(got[o]).max() == 0
    gotd = wc.matpc_sym(psi, dagger=True).reshape(-1)
    assert np.abs(gotd[e] - Sym.conj().T @ v).max() < 1e-13


def test_matpc_sym_solve_matches_full_system():
    """Solving the symmetric system with the symmetric source reconstructs the solution of
    the full M x = b (dense LU on 2^4), as the asymmetric form does."""
    dims = (2, 2, 2, 2)
    wc, M, e = _dense_system(dims, 73, 0.124, 1.0)
    b = qgen.spinor(dims, 74)
    xe, hist = oracle.bicgstab(wc.matpc_sym, wc.prepare_sym(b), tol=1e-14, maxiter=500)
    x = wc.reconstruct(xe, b)
    xlu = np.linalg.solve(M, b.reshape(-1))
    assert np.linalg.norm(x.reshape(-1) - xlu) / np.linalg.norm(xlu) < 1e-12


def test_matpc_gamma5_hermiticity_and_mdagm():
    """The asymmetric Schur form is gamma5-Hermitian: gamma5 Mhat gamma5 = Mhat^dag (explicit)."""
    dims = (4, 2, 2, 4)
    U = qgen.gauge(dims, 63)
    wc = oracle.WilsonClover(U, 0.12, 1.0)
    psi = oracle.restrict(qgen.spinor(dims, 64), 0)
    g5 = oracle.gamma5()
    g = lambda f: np.einsum("st,...tc->...sc", g5, f)
    lhs = g(wc.matpc(g(psi)))
    rhs = wc.matpc(psi, dagger=True)
    assert np.linalg.norm(lhs - rhs) / np.linalg.norm(rhs) < 1e-14
    phi = oracle.restrict(qgen.spinor(dims, 65), 0)
    a = np.vdot(phi, wc.matpc(psi))
    b = np.vdot(wc.matpc(phi, dagger=True), psi)
    assert abs(a - b) / abs(a) < 1e-14
    mm = wc.mdagm(psi)
    assert np.vdot(psi, mm).real > 0 and abs(np.vdot(psi, mm).imag) < 1e-10 * abs(np.vdot(psi, mm))


def test_free_field_matpc_closed_form():
    """Unit gauge (T = 1): Mhat psi_e = e^{ip.x}(1 - kappa^2 Dt(p)^2) u on even sites."""
    dims = (4, 4, 2, 4)
    kappa = 0.12
    wc = oracle.WilsonClover(qgen.unit_gauge(dims), kappa, 1.0, -1.0)
    u = RNG.normal(size=(4, 3)) + 1j * RNG.normal(size=(4, 3))
    p, pw = _plane_wave(dims, (1, 1, 0, 1), True, u)
    Dt = sum(2 * np.cos(p[m]) * np.eye(4) - 2j * np.sin(p[m]) * oracle.gamma(m) for m in range(4))
    psi_e = oracle.restrict(pw, 0)
    expect = oracle.restrict(np.einsum("st,...tc->...sc", np.eye(4) - kappa ** 2 * Dt @ Dt, pw), 0)
    assert np.abs(wc.matpc(psi_e) - expect).max() < 1e-13


def test_bicgstab_and_schur_solve_vs_lu():
    dims = (2, 2, 2, 2)
    wc, M, e = _dense_system(dims, 71, 0.124, 1.0)
    b = qgen.spinor(dims, 72)
    bh = wc.prepare(b)
    xe, hist = oracle.bicgstab(wc.matpc, bh, tol=1e-14, maxiter=500)
    assert hist[-1] <= 1e-14
    assert oracle.true_residual(wc.matpc, xe, bh) < 1e-13
    x = wc.reconstruct(xe, b)
    xlu = np.linalg.solve(M, b.reshape(-1))
    assert np.linalg.norm(x.reshape(-1) - xlu) / np.linalg.norm(xlu) < 1e-12
    # full-system residual of the reconstructed solution
    assert np.linalg.norm(M @ x.reshape(-1) - b.reshape(-1)) / np.linalg.norm(b) < 1e-12


def test_bicgstab_4x4_true_residual():
    dims = (4, 4, 4, 4)
    U = qgen.gauge(dims, 81, eps=0.1)
    wc = oracle.WilsonClover(U, 0.124, 1.0)
    b = qgen.point_source(dims, 0, 0)
    bh = wc.prepare(b)
    xe, hist = oracle.bicgstab(wc.matpc, bh, tol=1e-12, maxiter=1000)
    assert oracle.true_residual(wc.matpc, xe, bh) < 1e-11
    x = wc.reconstruct(xe, b)
    assert np.linalg.norm(wc.M(x) - b) / np.linalg.norm(b) < 1e-11


def test_sampled_evaluation_matches_full():
    """The site-sampled oracle (used at full BASELINE sizes) is the same per-site arithmetic:
    it must reproduce the full-lattice D, T and Mhat exactly at the sampled sites."""
    dims = (4, 4, 2, 6)
    U = qgen.gauge(dims, 91)
    psi = qgen.spinor(dims, 92)
    wc = oracle.WilsonClover(U, 0.12, 1.1, -1.0)
    rng = np.random.default_rng(3)
    sites = rng.choice(np.prod(dims), size=20, replace=False)
    full = oracle.dslash(U, psi, -1.0, True).reshape(-1, 4, 3)
    assert np.array_equal(oracle.dslash_sites(U, psi, sites, -1.0, True), full[sites])
    assert np.array_equal(oracle.clover_sites(U, sites, 0.12, 1.1), wc.T.reshape(-1, 12, 12)[sites])
    odd = oracle.parity_mask(dims).reshape(-1)
    ev = np.nonzero(~odd)[0][::3]
    psi_e = oracle.restrict(psi, 0)
    got = oracle.matpc_sites(U, psi_e, ev, 0.12, 1.1, -1.0)
    want = wc.matpc(psi_e).reshape(-1, 4, 3)[ev]
    assert np.abs(got - want).max() < 1e-13


@pytest.mark.parametrize("chunk", [7, 13, 1 << 17])
def test_apply_M_chunked_pins(chunk):
    """oracle.apply_M_chunked (the full-size residual checker, T evaluated chunk by chunk with
    clover_sites) against (i) the closed form on the unit gauge, where T = 1 and M_kappa =
    1 - kappa D acts on a plane wave as e^{ip.x}(1 - kappa sum_mu (2 cos p_mu - 2 i gamma_mu
    sin p_mu)) u (reading Q4; no oracle involved), and (ii) T - kappa D from the
    whole-lattice clover (WilsonClover.M, pinned above by the abelian closed form and the dense
    Schur complement) at odd chunk sizes that cut the lattice mid-timeslice.  Catches a dropped
    chunk tail, a wrong -kappa sign, or the clover applied to the wrong sites."""
    dims = (4, 4, 2, 6)
    kappa, csw = 0.124, 1.0
    u = RNG.normal(size=(4, 3)) + 1j * RNG.normal(size=(4, 3))
    for antiperiodic in (True, False):
        p, pw = _plane_wave(dims, (1, 1, 0, 2), antiperiodic, u)
        Dt = sum(2 * np.cos(p[m]) * np.eye(4) - 2j * np.sin(p[m]) * oracle.gamma(m) for m in range(4))
        expect = np.einsum("st,...tc->...sc", np.eye(4) - kappa * Dt, pw)
        got = oracle.apply_M_chunked(qgen.unit_gauge(dims), pw, kappa, csw, -1.0 if antiperiodic else 1.0, chunk=chunk)
        assert np.abs(got - expect).max() < 1e-13
    U = qgen.gauge(dims, 93)
    x = qgen.spinor(dims, 94)
    wc = oracle.WilsonClover(U, kappa, csw, -1.0)
    got = oracle.apply_M_chunked(U, x, kappa, csw, -1.0, chunk=chunk)
    assert np.abs(got - wc.M(x)).max() < 1e-13 * np.abs(wc.M(x)).max()
