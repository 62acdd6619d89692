"""CPU oracle for the ArrayOL HD->SD downscaler -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline``
/ ``--impl reference`` legs may import this package.  The product path
(``paper_conf_ipps_guortgbs11_b200``) never imports it and shares no code with
it.  The arithmetic lives in plain C (``aol_oracle.c``); this module only
marshals numpy arrays through ctypes.

Every function follows /root/reference/PAPER.md literally; see
``aol_oracle.h`` for the per-function citations and pins.  The vertical
filter is the reading Z1/Z2 of DESIGN.md ("parity pinned by invariants only":
the paper never prints the V tiler).
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_LIB = None

MAX_RANK = 8
PRESET_H_IN, PRESET_H_OUT, PRESET_V_IN, PRESET_V_OUT = 0, 1, 2, 3


class Tiler(ctypes.Structure):
    """oracle_tiler (aol_oracle.h); Fig. 10 record, matrices [array_dim][col]."""

    _fields_ = [
        ("array_rank", ctypes.c_int32),
        ("rep_rank", ctypes.c_int32),
        ("pattern_rank", ctypes.c_int32),
        ("array_shape", ctypes.c_int64 * MAX_RANK),
        ("rep_shape", ctypes.c_int64 * MAX_RANK),
        ("pattern_shape", ctypes.c_int64 * MAX_RANK),
        ("origin", ctypes.c_int64 * MAX_RANK),
        ("paving", (ctypes.c_int64 * MAX_RANK) * MAX_RANK),
        ("fitting", (ctypes.c_int64 * MAX_RANK) * MAX_RANK),
    ]

    @property
    def shapes(self):
        a = tuple(self.array_shape[k] for k in range(self.array_rank))
        r = tuple(self.rep_shape[k] for k in range(self.rep_rank))
        p = tuple(self.pattern_shape[k] for k in range(self.pattern_rank))
        return a, r, p


def build(force: bool = False) -> str:
    """Compile liboracle.so with gcc (plain C99, -O2, OpenMP across planes)."""
    src = os.path.join(_HERE, "aol_oracle.c")
    hdr = os.path.join(_HERE, "aol_oracle.h")
    if (not force and os.path.exists(_SO)
            and os.path.getmtime(_SO) >= max(os.path.getmtime(src), os.path.getmtime(hdr))):
        return _SO
    tmp = _SO + f".tmp{os.getpid()}"
    subprocess.check_call(["gcc", "-std=c99", "-O2", "-fopenmp", "-fPIC", "-shared",
                           "-Wall", "-Wextra", "-o", tmp, src])
    os.replace(tmp, _SO)
    return _SO


def lib():
    global _LIB
    if _LIB is None:
        build()
        L = ctypes.CDLL(_SO)
        P = ctypes.c_void_p
        i64 = ctypes.c_int64
        TP = ctypes.POINTER(Tiler)
        sigs = {
            "oracle_tiler_preset": [ctypes.c_int, i64, i64, TP],
            "oracle_gather": [TP, ctypes.c_int, P, P],
            "oracle_scatter": [TP, ctypes.c_int, P, P],
            "oracle_task_h": [P, i64, P],
            "oracle_task_v": [P, i64, P],
            "oracle_downscale_h": [P, P, i64, i64],
            "oracle_downscale_v": [P, P, i64, i64],
            "oracle_downscale_frame": [P, P, i64, i64, i64, i64, P, ctypes.c_int],
            "oracle_checksum": [P, i64, i64, i64, i64, P],
            "oracle_max_threads": [],
        }
        for name, args in sigs.items():
            f = getattr(L, name)
            f.argtypes = args
            f.restype = ctypes.c_int
        _LIB = L
    return _LIB


def _ptr(a: np.ndarray):
    return a.ctypes.data_as(ctypes.c_void_p)


def _check(rc: int, what: str):
    if rc != 0:
        raise ValueError(f"oracle {what} rejected its arguments (rc={rc})")


def make_tiler(array_shape, rep_shape, pattern_shape, origin=None, paving=None, fitting=None) -> Tiler:
    """Build a tiler; paving is [array_rank][rep_rank], fitting [array_rank][pattern_rank]."""
    t = Tiler()
    ra, rr, rp = len(array_shape), len(rep_shape), len(pattern_shape)
    t.array_rank, t.rep_rank, t.pattern_rank = ra, rr, rp
    for k, v in enumerate(array_shape):
        t.array_shape[k] = int(v)
    for k, v in enumerate(rep_shape):
        t.rep_shape[k] = int(v)
    for k, v in enumerate(pattern_shape):
        t.pattern_shape[k] = int(v)
    for a in range(ra):
        t.origin[a] = int(origin[a]) if origin is not None else 0
        for j in range(rr):
            t.paving[a][j] = int(paving[a][j]) if paving is not None else 0
        for k in range(rp):
            t.fitting[a][k] = int(fitting[a][k]) if fitting is not None else 0
    return t


def preset(which: int, H: int, W: int) -> Tiler:
    t = Tiler()
    _check(lib().oracle_tiler_preset(which, H, W, ctypes.byref(t)), "preset")
    return t


def gather(t: Tiler, A: np.ndarray) -> np.ndarray:
    A = np.ascontiguousarray(A)
    arr, rep, pat = t.shapes
    assert A.shape == arr, (A.shape, arr)
    G = np.empty(rep + pat, dtype=A.dtype)
    _check(lib().oracle_gather(ctypes.byref(t), A.itemsize, _ptr(A), _ptr(G)), "gather")
    return G


def scatter(t: Tiler, G: np.ndarray, A: np.ndarray) -> np.ndarray:
    """Return a copy of A with G scattered in (Fig. 6 order; A itself is untouched)."""
    arr, rep, pat = t.shapes
    G = np.require(G, requirements="C")       # keeps 0-d arrays 0-d
    assert G.shape == rep + pat and A.shape == arr and G.dtype == A.dtype
    out = np.array(A, copy=True, order="C")
    _check(lib().oracle_scatter(ctypes.byref(t), out.itemsize, _ptr(G), _ptr(out)), "scatter")
    return out


def task_h(G: np.ndarray) -> np.ndarray:
    G = np.ascontiguousarray(G, dtype=np.int32)
    assert G.shape[-1] == 11
    T = np.empty(G.shape[:-1] + (3,), np.int32)
    _check(lib().oracle_task_h(_ptr(G), G.size // 11, _ptr(T)), "task_h")
    return T


def task_v(G: np.ndarray) -> np.ndarray:
    G = np.ascontiguousarray(G, dtype=np.int32)
    assert G.shape[-1] == 12
    T = np.empty(G.shape[:-1] + (4,), np.int32)
    _check(lib().oracle_task_v(_ptr(G), G.size // 12, _ptr(T)), "task_v")
    return T


def downscale_h(X: np.ndarray) -> np.ndarray:
    """One plane (H, W) or a stack (..., H, W) -> (..., H, 3W/8)."""
    X = np.ascontiguousarray(X, dtype=np.int32)
    H, W = X.shape[-2:]
    Y = np.empty(X.shape[:-1] + (3 * (W // 8),), np.int32)
    Xp, Yp = X.reshape(-1, H, W), Y.reshape(-1, H, 3 * (W // 8))
    for p in range(Xp.shape[0]):
        _check(lib().oracle_downscale_h(_ptr(Xp[p]), _ptr(Yp[p]), H, W), "downscale_h")
    return Y


def downscale_v(Y: np.ndarray) -> np.ndarray:
    """One plane (H, Wo) or a stack (..., H, Wo) -> (..., 4H/9, Wo)."""
    Y = np.ascontiguousarray(Y, dtype=np.int32)
    H, Wo = Y.shape[-2:]
    Z = np.empty(Y.shape[:-2] + (4 * (H // 9), Wo), np.int32)
    Yp, Zp = Y.reshape(-1, H, Wo), Z.reshape(-1, 4 * (H // 9), Wo)
    for p in range(Yp.shape[0]):
        _check(lib().oracle_downscale_v(_ptr(Yp[p]), _ptr(Zp[p]), H, Wo), "downscale_v")
    return Z


def downscale_frame(X: np.ndarray, nthreads: int = 1):
    """X [frames][channels][H][W] int32 -> (Z [frames][channels][4H/9][3W/8], checksums u64[frames])."""
    X = np.ascontiguousarray(X, dtype=np.int32)
    N, C, H, W = X.shape
    Z = np.empty((N, C, 4 * (H // 9), 3 * (W // 8)), np.int32)
    cs = np.empty(N, np.uint64)
    _check(lib().oracle_downscale_frame(_ptr(X), _ptr(Z), N, C, H, W, _ptr(cs), int(nthreads)),
           "downscale_frame")
    return Z, cs


def checksum(Z: np.ndarray) -> np.ndarray:
    Z = np.ascontiguousarray(Z, dtype=np.int32)
    N, C, Ho, Wo = Z.shape
    cs = np.empty(N, np.uint64)
    _check(lib().oracle_checksum(_ptr(Z), N, C, Ho, Wo, _ptr(cs)), "checksum")
    return cs


def max_threads() -> int:
    return int(lib().oracle_max_threads())
