"""Oracle — TEST INFRASTRUCTURE ONLY (fp64, CPU, plain and slow).

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference legs
may import this package.  It shares no code with the CUDA product path
(paper_1011_0024_b200/) and never imports it; the product never imports this.

What it computes, in the paper's notation (PAPER.md = arXiv:1011.0024 text):
  D        eq. (2), P:152-162 — oracle.c: oracle_dslash (full 4x4 gammas, 3x3 links)
  A, T     eq. (2) clover, P:167-169 + footnote 1 P:183-184 — oracle.c: oracle_clover
           (reading Q1: four-leaf SW clover; T = 1 + 2 kappa A)
  M_kappa  = 2 kappa M(eq. 2) = T - kappa D  (reading Q4, kappa = 1/(2(4+m)))
  Mhat     even-odd Schur complement, P:190-195 (reading Q2, asymmetric, even sites):
           Mhat = T_ee - kappa^2 D_eo T_oo^{-1} D_oe ; its adjoint by the EXPLICIT formula
           Mhat^dag = T_ee - kappa^2 (D^dag)_eo T_oo^{-1} (D^dag)_oe
  prepare / reconstruct  b_hat = b_e + kappa D_eo T_oo^{-1} b_o ;
           x_o = T_oo^{-1} (b_o + kappa D_oe x_e)
  bicgstab textbook BiCGstab of van der Vorst (ref [8]), fp64,
           no reliable updates, residual history recorded.
  dense_*  brute-force dense matrices on tiny lattices, built entry by entry from eq. (2)
           with index logic independent of oracle.c (pins, not the oracle proper).

Field conventions: gauge U[4, T, Z, Y, X, 3, 3] (mu = x, y, z, t); spinor psi[T, Z, Y, X,
4, 3] in the DeGrand-Rossi basis; parity of a site = (x + y + z + t) mod 2 (reading Q14);
a "parity field" is a full-lattice array that is zero on the other parity.

Parity status: every function here is pinned by tests/test_oracle_pins.py (DESIGN.md §3 lists
each function with its pin; apply_M_chunked by test_apply_M_chunked_pins); none is "parity
unpinned".
"""
import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "_oracle.so")
_lib = None


def build(force=False):
    src = os.path.join(_HERE, "oracle.c")
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < os.path.getmtime(src):
        subprocess.check_call(["gcc", "-O2", "-fopenmp", "-fPIC", "-shared", "-o", _SO, src, "-lm"])
    return _SO


def _load():
    global _lib
    if _lib is None:
        build()
        _lib = ctypes.CDLL(_SO)
        dp = ctypes.POINTER(ctypes.c_double)
        ip = ctypes.POINTER(ctypes.c_int)
        _lib.oracle_gamma.argtypes = [ctypes.c_int, dp]
        _lib.oracle_dslash.argtypes = [dp, dp, dp, ip, ctypes.c_double, ctypes.c_int, ctypes.c_int, ctypes.c_int]
        _lib.oracle_clover.argtypes = [dp, dp, ip, ctypes.c_double, ctypes.c_double]
        _lib.oracle_invert12.argtypes = [dp, dp, ctypes.c_long]
        _lib.oracle_invert12.restype = ctypes.c_int
        _lib.oracle_site_mult.argtypes = [dp, dp, dp, ctypes.c_long]
        lp = ctypes.POINTER(ctypes.c_long)
        _lib.oracle_dslash_sites.argtypes = [dp, dp, dp, ip, ctypes.c_double, ctypes.c_int, lp, ctypes.c_long]
        _lib.oracle_clover_sites.argtypes = [dp, dp, ip, ctypes.c_double, ctypes.c_double, lp, ctypes.c_long]
    return _lib


def _p(a):
    assert a.dtype == np.complex128 and a.flags.c_contiguous
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_double))


def _dims_of_spinor(psi):
    T, Z, Y, X = psi.shape[:4]
    return (X, Y, Z, T)


def _cdims(dims):
    return (ctypes.c_int * 4)(*[int(d) for d in dims])


def set_threads(n):
    """OpenMP thread count for the C oracle (must be called before the first call)."""
    os.environ["OMP_NUM_THREADS"] = str(int(n))


# ----------------------------------------------------------------------------- gamma

def gamma(mu):
    """gamma_mu (mu = 0..3 for x, y, z, t) in the DeGrand-Rossi basis, 4x4 complex."""
    out = np.empty((4, 4), dtype=np.complex128)
    _load().oracle_gamma(int(mu), _p(out))
    return out


def gamma5():
    return gamma(0) @ gamma(1) @ gamma(2) @ gamma(3)


# ----------------------------------------------------------------------------- operator

def dslash(U, psi, t_bc=-1.0, dagger=False, t_global_offset=0, T_global=None):
    """D psi (eq. 2) or the explicit adjoint D^dag psi, every site; periodic array with
    the temporal boundary factor t_bc on hops crossing global t = T-1 <-> 0."""
    dims = _dims_of_spinor(psi)
    U = np.ascontiguousarray(U)
    psi = np.ascontiguousarray(psi)
    out = np.empty_like(psi)
    Tg = dims[3] if T_global is None else T_global
    _load().oracle_dslash(_p(out), _p(U), _p(psi), _cdims(dims), float(t_bc), int(bool(dagger)),
                          int(t_global_offset), int(Tg))
    return out


def clover(U, kappa, csw):
    """T(x) = 1 + 2 kappa A(x), shape [T, Z, Y, X, 12, 12] (index s*3 + colour)."""
    U = np.ascontiguousarray(U)
    T_, Z, Y, X = U.shape[1:5]
    out = np.empty((T_, Z, Y, X, 12, 12), dtype=np.complex128)
    _load().oracle_clover(_p(out), _p(U), _cdims((X, Y, Z, T_)), float(kappa), float(csw))
    return out


def invert12(Tm):
    Tm = np.ascontiguousarray(Tm)
    out = np.empty_like(Tm)
    V = int(np.prod(Tm.shape[:-2]))
    bad = _load().oracle_invert12(_p(out), _p(Tm), V)
    if bad:
        raise ArithmeticError(f"oracle_invert12: {bad} singular site matrices")
    return out


def site_mult(M, psi):
    M = np.ascontiguousarray(M)
    psi = np.ascontiguousarray(psi)
    out = np.empty_like(psi)
    V = int(np.prod(psi.shape[:4]))
    _load().oracle_site_mult(_p(out), _p(M), _p(psi), V)
    return out


def parity_mask(dims):
    """Boolean [T, Z, Y, X], True on odd sites ((x+y+z+t) mod 2 == 1)."""
    X, Y, Z, T = dims
    t, z, y, x = np.meshgrid(np.arange(T), np.arange(Z), np.arange(Y), np.arange(X), indexing="ij")
    return ((x + y + z + t) % 2) == 1


def restrict(psi, parity):
    """Zero the sites of the other parity."""
    m = parity_mask(_dims_of_spinor(psi))
    keep = m if parity == 1 else ~m
    out = psi.copy()
    out[~keep] = 0
    return out


class WilsonClover:
    """The even-odd preconditioned Wilson-clover system on one global lattice."""

    def __init__(self, U, kappa, csw, t_bc=-1.0):
        self.U = np.ascontiguousarray(U)
        self.kappa = float(kappa)
        self.csw = float(csw)
        self.t_bc = float(t_bc)
        self.T = clover(self.U, kappa, csw)
        self.Tinv = invert12(self.T)

    # full operator M_kappa = T - kappa D
    def D(self, psi, dagger=False):
        return dslash(self.U, psi, self.t_bc, dagger)

    def M(self, psi, dagger=False):
        return site_mult(self.T, psi) - self.kappa * self.D(psi, dagger)

    # even-odd pieces: D_{p,1-p} psi = restrict(D restrict(psi, 1-p), p)
    def Dpq(self, psi, out_parity, dagger=False):
        return restrict(self.D(restrict(psi, 1 - out_parity), dagger), out_parity)

    def Tpp(self, psi, parity):
        return restrict(site_mult(self.T, psi), parity)

    def Tinv_pp(self, psi, parity):
        return restrict(site_mult(self.Tinv, psi), parity)

    def matpc(self, x_e, dagger=False):
        """Mhat x_e = T_ee x_e - kappa^2 D_eo T_oo^{-1} D_oe x_e (even sites);
        dagger: the explicit adjoint T_ee - kappa^2 (D^dag)_eo T_oo^-1 (D^dag)_oe."""
        tmp = self.Tinv_pp(self.Dpq(x_e, 1, dagger), 1)
        return self.Tpp(x_e, 0) - self.kappa ** 2 * self.Dpq(tmp, 0, dagger)

    def mdagm(self, x_e):
        return self.matpc(self.matpc(x_e), dagger=True)

    def matpc_sym(self, x_e, dagger=False):
        """Symmetric Schur complement (the other form of P:190-195):
        Mhat_sym x_e = x_e - kappa^2 T_ee^{-1} D_eo T_oo^{-1} D_oe x_e (even sites), i.e.
        T_ee^{-1} (M_ee - M_eo M_oo^{-1} M_oe).  dagger: the explicit adjoint
        x_e - kappa^2 (D^dag)_eo T_oo^{-1} (D^dag)_oe T_ee^{-1} x_e (T Hermitian)."""
        if not dagger:
            tmp = self.Tinv_pp(self.Dpq(x_e, 1), 1)
            return restrict(x_e, 0) - self.kappa ** 2 * self.Tinv_pp(self.Dpq(tmp, 0), 0)
        y = self.Tinv_pp(x_e, 0)
        tmp = self.Tinv_pp(self.Dpq(y, 1, True), 1)
        return restrict(x_e, 0) - self.kappa ** 2 * self.Dpq(tmp, 0, True)

    def prepare_sym(self, b):
        """Source of the symmetric system: T_ee^{-1} (b_e + kappa D_eo T_oo^{-1} b_o)."""
        return self.Tinv_pp(self.prepare(b), 0)

    def prepare(self, b):
        b_e, b_o = restrict(b, 0), restrict(b, 1)
        return b_e + self.kappa * self.Dpq(self.Tinv_pp(b_o, 1), 0)

    def reconstruct(self, x_e, b):
        b_o = restrict(b, 1)
        x_o = self.Tinv_pp(b_o + self.kappa * self.Dpq(x_e, 1), 1)
        return x_e + x_o


# ----------------------------------------------------------------------------- sampled sites
# For lattices too large to evaluate everywhere (BASELINE full sizes), the same per-site
# arithmetic as dslash()/clover() (oracle.c: dslash_one / clover_one) evaluated at a list of
# lexicographic site indices of the global lattice.

def _sites_arr(sites):
    s = np.ascontiguousarray(np.asarray(sites, dtype=np.int64))
    return s, s.ctypes.data_as(ctypes.POINTER(ctypes.c_long))


def dslash_sites(U, psi, sites, t_bc=-1.0, dagger=False):
    """(D psi)(x) for x in sites; returns [len(sites), 4, 3]."""
    dims = _dims_of_spinor(psi)
    s, sp = _sites_arr(sites)
    out = np.empty((len(s), 4, 3), dtype=np.complex128)
    _load().oracle_dslash_sites(_p(out), _p(np.ascontiguousarray(U)), _p(np.ascontiguousarray(psi)), _cdims(dims),
                                float(t_bc), int(bool(dagger)), sp, len(s))
    return out


def clover_sites(U, sites, kappa, csw):
    T_, Z, Y, X = U.shape[1:5]
    s, sp = _sites_arr(sites)
    out = np.empty((len(s), 12, 12), dtype=np.complex128)
    _load().oracle_clover_sites(_p(out), _p(np.ascontiguousarray(U)), _cdims((X, Y, Z, T_)), float(kappa),
                                float(csw), sp, len(s))
    return out


def neighbours(dims, sites):
    """The 8 nearest neighbours (lex indices) of each site, shape [n, 8]."""
    X, Y, Z, T = dims
    s = np.asarray(sites, dtype=np.int64)
    c = [s % X, (s // X) % Y, (s // (X * Y)) % Z, s // (X * Y * Z)]
    L = [X, Y, Z, T]
    out = []
    for mu in range(4):
        for step in (1, -1):
            n = [ci.copy() for ci in c]
            n[mu] = (n[mu] + step) % L[mu]
            out.append(((n[3] * Z + n[2]) * Y + n[1]) * X + n[0])
    return np.stack(out, axis=1)


def apply_M_chunked(U, x, kappa, csw, t_bc=-1.0, chunk=1 << 17):
    """M_kappa x = T x - kappa D x on the whole lattice without storing the 12x12 clover of
    every site (T is evaluated chunk by chunk with clover_sites): for full-size residuals."""
    dims = _dims_of_spinor(x)
    out = -kappa * dslash(U, x, t_bc)
    xf = x.reshape(-1, 12)
    of = out.reshape(-1, 12)
    V = xf.shape[0]
    for s0 in range(0, V, chunk):
        idx = np.arange(s0, min(V, s0 + chunk))
        of[idx] += np.einsum("nij,nj->ni", clover_sites(U, idx, kappa, csw), xf[idx])
    return out


def matpc_sites(U, psi_e, sites, kappa, csw, t_bc=-1.0, dagger=False):
    """(Mhat psi_e)(x) for even sites x, Mhat = T_ee - kappa^2 D_eo T_oo^{-1} D_oe, evaluated
    only where needed: D_oe psi_e at the odd neighbours of the sample, T^{-1} there, then D_eo at
    the sample.  psi_e: full-lattice array zero on odd sites."""
    dims = _dims_of_spinor(psi_e)
    sites = np.asarray(sites, dtype=np.int64)
    nb = np.unique(neighbours(dims, sites).ravel())
    d_nb = dslash_sites(U, psi_e, nb, t_bc, dagger)
    tinv = invert12(clover_sites(U, nb, kappa, csw))
    tmp = np.zeros_like(psi_e)
    tmp.reshape(-1, 4, 3)[nb] = np.einsum("nij,nj->ni", tinv, d_nb.reshape(-1, 12)).reshape(-1, 4, 3)
    dd = dslash_sites(U, tmp, sites, t_bc, dagger)
    Tx = clover_sites(U, sites, kappa, csw)
    tx = np.einsum("nij,nj->ni", Tx, psi_e.reshape(-1, 12)[sites]).reshape(-1, 4, 3)
    return tx - kappa ** 2 * dd


# ----------------------------------------------------------------------------- solver

def vdot(a, b):
    return complex(np.vdot(a.ravel(), b.ravel()))


def norm(a):
    return float(np.linalg.norm(a.ravel()))


def bicgstab(A, b, tol=1e-12, maxiter=10000, x0=None):
    """Textbook BiCGstab (van der Vorst 1992, ref [8]).  Returns (x, history) with
    history = list of ||r_k|| / ||b|| for the recursively updated residual."""
    x = np.zeros_like(b) if x0 is None else x0.copy()
    r = b - A(x) if x0 is not None else b.copy()
    rhat = r.copy()
    rho = alpha = omega = 1.0 + 0j
    v = np.zeros_like(b)
    p = np.zeros_like(b)
    bnorm = norm(b)
    hist = []
    for _ in range(maxiter):
        rho_new = vdot(rhat, r)
        beta = (rho_new / rho) * (alpha / omega)
        p = r + beta * (p - omega * v)
        v = A(p)
        alpha = rho_new / vdot(rhat, v)
        s = r - alpha * v
        t = A(s)
        omega = vdot(t, s) / vdot(t, t)
        x = x + alpha * p + omega * s
        r = s - omega * t
        rho = rho_new
        hist.append(norm(r) / bnorm)
        if hist[-1] <= tol:
            break
    return x, hist


def true_residual(A, x, b):
    """||b - A x|| / ||b|| in fp64."""
    return norm(b - A(x)) / norm(b)


# ----------------------------------------------------------------------------- dense pins

def dense_hopping(U, t_bc=-1.0):
    """Dense D (eq. 2) on a tiny lattice, built entry by entry.  Index logic is written
    independently of oracle.c: sites enumerated by coordinate tuples, matrix index
    (site, spin, colour) with site = x + X*(y + Y*(z + Z*t))."""
    _, T, Z, Y, X = U.shape[:5]
    L = (X, Y, Z, T)
    g = [gamma(mu) for mu in range(4)]
    one = np.eye(4)
    V = X * Y * Z * T
    N = 12 * V

    def idx(c):
        x, y, z, t = (c[0] % X, c[1] % Y, c[2] % Z, c[3] % T)
        return x + X * (y + Y * (z + Z * t))

    def link(mu, c):
        x, y, z, t = (c[0] % X, c[1] % Y, c[2] % Z, c[3] % T)
        return U[mu, t, z, y, x]

    Dm = np.zeros((N, N), dtype=np.complex128)
    for t in range(T):
        for z in range(Z):
            for y in range(Y):
                for x in range(X):
                    c = (x, y, z, t)
                    i = idx(c)
                    for mu in range(4):
                        cf = list(c); cf[mu] += 1
                        cb = list(c); cb[mu] -= 1
                        fsign = t_bc if (mu == 3 and t == T - 1) else 1.0
                        bsign = t_bc if (mu == 3 and t == 0) else 1.0
                        blk_f = fsign * np.kron(one - g[mu], link(mu, c))
                        blk_b = bsign * np.kron(one + g[mu], link(mu, cb).conj().T)
                        jf, jb = idx(cf), idx(cb)
                        Dm[12 * i:12 * i + 12, 12 * jf:12 * jf + 12] += blk_f
                        Dm[12 * i:12 * i + 12, 12 * jb:12 * jb + 12] += blk_b
    return Dm


def to_dense_vec(psi):
    """[T, Z, Y, X, 4, 3] -> dense vector in dense_hopping's index order (identical: site
    index x + X(y + Y(z + Z t)) is the C-order flattening of [t, z, y, x])."""
    return psi.reshape(-1).copy()


def from_dense_vec(v, dims):
    X, Y, Z, T = dims
    return v.reshape(T, Z, Y, X, 4, 3)
