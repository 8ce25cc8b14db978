"""Seeded synthetic inputs (shared by oracle-side and CUDA-side tests, bench, smoke).

Holds none of the method's arithmetic — it draws random numbers and builds the input
fields of the paper's experiments (weak-field SU(3) links; Haar
links; Gaussian spinors; point sources).  See qgen.c for the counter scheme.

Arrays are numpy complex128:
  gauge  : [4, nt, Z, Y, X, 3, 3]   (mu, t, z, y, x, row, col)
  spinor : [nt, Z, Y, X, 4, 3]      (t, z, y, x, spin, colour), DeGrand-Rossi basis
"""
import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "_qgen.so")
_lib = None


def build(force=False):
    src = os.path.join(_HERE, "qgen.c")
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
        _lib.qgen_gauge.argtypes = [dp, ip, ctypes.c_int, ctypes.c_int, ctypes.c_uint64, ctypes.c_double]
        _lib.qgen_spinor.argtypes = [dp, ip, ctypes.c_int, ctypes.c_int, ctypes.c_uint64]
        _lib.qgen_gauge_transform.argtypes = [dp, ip, ctypes.c_int, ctypes.c_int, ctypes.c_uint64]
        _lib.qgen_gauge_box.argtypes = [dp, ip, ip, ip, ctypes.c_uint64, ctypes.c_double]
        _lib.qgen_spinor_box.argtypes = [dp, ip, ip, ip, ctypes.c_uint64]
    return _lib


def _dims(dims):
    return (ctypes.c_int * 4)(*[int(d) for d in dims])


def _ptr(a):
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_double))


def gauge(dims, seed, eps=-1.0, t_begin=0, nt=None):
    """SU(3) gauge field on timeslices t_begin..t_begin+nt-1 (mod T) of the global lattice
    dims = (X, Y, Z, T).  eps < 0: Haar links; eps >= 0: weak field 1 + eps*noise,
    re-unitarised."""
    X, Y, Z, T = dims
    nt = T if nt is None else nt
    out = np.empty((4, nt, Z, Y, X, 3, 3), dtype=np.complex128)
    _load().qgen_gauge(_ptr(out), _dims(dims), int(t_begin), int(nt), int(seed), float(eps))
    return out


def spinor(dims, seed, t_begin=0, nt=None):
    """Gaussian colour-spinor field (unit variance per real component)."""
    X, Y, Z, T = dims
    nt = T if nt is None else nt
    out = np.empty((nt, Z, Y, X, 4, 3), dtype=np.complex128)
    _load().qgen_spinor(_ptr(out), _dims(dims), int(t_begin), int(nt), int(seed))
    return out


def gauge_box(dims, seed, origin, extent, eps=-1.0):
    """gauge() restricted to the box origin .. origin + extent (x, y, z, t order) of the global
    lattice: [4, et, ez, ey, ex, 3, 3] — the same values as the corresponding slice of gauge()."""
    ex, ey, ez, et = extent
    out = np.empty((4, et, ez, ey, ex, 3, 3), dtype=np.complex128)
    _load().qgen_gauge_box(_ptr(out), _dims(dims), _dims(origin), _dims(extent), int(seed), float(eps))
    return out


def spinor_box(dims, seed, origin, extent):
    """spinor() restricted to a box: [et, ez, ey, ex, 4, 3]."""
    ex, ey, ez, et = extent
    out = np.empty((et, ez, ey, ex, 4, 3), dtype=np.complex128)
    _load().qgen_spinor_box(_ptr(out), _dims(dims), _dims(origin), _dims(extent), int(seed))
    return out


def gauge_transform(dims, seed, t_begin=0, nt=None):
    """Haar SU(3) gauge transformation G(x), shape [nt, Z, Y, X, 3, 3]."""
    X, Y, Z, T = dims
    nt = T if nt is None else nt
    out = np.empty((nt, Z, Y, X, 3, 3), dtype=np.complex128)
    _load().qgen_gauge_transform(_ptr(out), _dims(dims), int(t_begin), int(nt), int(seed))
    return out


def point_source(dims, spin, colour, site=(0, 0, 0, 0), t_begin=0, nt=None):
    """Unit point source at global site (x, y, z, t), spin/colour component — the
    6 sources of the paper's tests are colour 0-2 x spin 0-1."""
    X, Y, Z, T = dims
    nt = T if nt is None else nt
    out = np.zeros((nt, Z, Y, X, 4, 3), dtype=np.complex128)
    x, y, z, t = site
    tl = (t - t_begin) % T
    if tl < nt:
        out[tl, z, y, x, spin, colour] = 1.0
    return out


def unit_gauge(dims):
    X, Y, Z, T = dims
    out = np.zeros((4, T, Z, Y, X, 3, 3), dtype=np.complex128)
    for a in range(3):
        out[..., a, a] = 1.0
    return out
