"""Seeded synthetic frame generator (host side, numpy).

This module holds NO arithmetic of the method.  It stands in for the paper's
FrameGenerator IP, which reads real video through OpenCV (
out of scope, the videos are unnamed).  Frames are planar int32
[frames][channels][H][W] (reading Z7/Z8 of DESIGN.md: three per-channel planes,
P:L671-675; 8-bit channel values).

Counter-based so that any element can be produced independently: the CUDA
library implements the SAME generator in its own code (``aol_synth_frames``),
and a GPU test checks the two agree bit for bit.  The oracle side always takes
its inputs from this module; the GPU side may use either.

    counter(seed, n, c, y, x) = seed * PHI + ((n*C + c)*H + y)*W + x     (mod 2**64)
    u = splitmix64(counter)
    uniform  : u >> 56                      -> [0, 255]   (24-bit RGB content)
    dark     : u >> 61                      -> [0, 7]     (drives V sums negative)
    signed   : (u >> 37) - 2**26            -> [-2**26, 2**26)  (inside the Z12 domain)
    ramp     : x                            (column index; closed-form pin)
    constant : value                        (invariant pin)

``n`` is the GLOBAL frame index (``frame0 + local index``), so a shard or a
sampled frame regenerates exactly the frame the full stream holds.

``frames_c`` is the same generator in plain C with OpenMP (``synth.c`` ->
``libsynth.so``): bench-size inputs (300 HD frames, 1.87 G samples) for the
oracle in well under a second.  tests/test_synth.py checks it equals ``frames``.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

PHI = np.uint64(0x9E3779B97F4A7C15)
_M1 = np.uint64(0xBF58476D1CE4E5B9)
_M2 = np.uint64(0x94D049BB133111EB)

KINDS = ("uniform", "dark", "signed", "ramp", "constant")
KIND_CODE = {k: i for i, k in enumerate(KINDS)}


def splitmix64(z: np.ndarray) -> np.ndarray:
    """Steele/Lea/Flood SplitMix64 finaliser applied to counters (uint64, wrapping)."""
    with np.errstate(over="ignore"):
        z = z + PHI
        z = (z ^ (z >> np.uint64(30))) * _M1
        z = (z ^ (z >> np.uint64(27))) * _M2
        return z ^ (z >> np.uint64(31))


def frames(seed: int, frame0: int, nframes: int, channels: int, H: int, W: int,
           kind: str = "uniform", value: int = 0) -> np.ndarray:
    """Return int32 [nframes][channels][H][W] for global frames frame0 .. frame0+nframes-1."""
    if kind not in KIND_CODE:
        raise ValueError(f"unknown kind {kind!r}; one of {KINDS}")
    shape = (nframes, channels, H, W)
    if kind == "ramp":
        return np.ascontiguousarray(np.broadcast_to(np.arange(W, dtype=np.int32), shape))
    if kind == "constant":
        return np.full(shape, value, dtype=np.int32)
    out = np.empty(shape, dtype=np.int32)
    plane = H * W
    lin = np.arange(plane, dtype=np.uint64)
    with np.errstate(over="ignore"):
        base_seed = np.uint64(seed & 0xFFFFFFFFFFFFFFFF) * PHI
        for f in range(nframes):
            for c in range(channels):
                start = np.uint64(((frame0 + f) * channels + c) * plane & 0xFFFFFFFFFFFFFFFF)
                u = splitmix64(base_seed + start + lin)
                if kind == "uniform":
                    v = (u >> np.uint64(56)).astype(np.int32)
                elif kind == "dark":
                    v = (u >> np.uint64(61)).astype(np.int32)
                else:  # signed
                    v = (u >> np.uint64(37)).astype(np.int64) - (1 << 26)
                out[f, c] = v.reshape(H, W).astype(np.int32)
    return out


def planes(seed: int, nplanes: int, H: int, W: int, kind: str = "uniform", value: int = 0) -> np.ndarray:
    """Convenience: [nplanes][H][W] (one channel per 'frame')."""
    return frames(seed, 0, nplanes, 1, H, W, kind, value)[:, 0]


# ---------------------------------------------------------------- C + OpenMP version (synth.c)

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "libsynth.so")
_LIB = None


def build(force: bool = False) -> str:
    """Compile libsynth.so with gcc (plain C99, -O2, OpenMP over rows)."""
    src = os.path.join(_HERE, "synth.c")
    if not force and os.path.exists(_SO) and os.path.getmtime(_SO) >= os.path.getmtime(src):
        return _SO
    tmp = _SO + f".tmp{os.getpid()}"
    subprocess.check_call(["gcc", "-std=c99", "-O2", "-fopenmp", "-fPIC", "-shared", "-Wall", "-Wextra",
                           "-o", tmp, src])
    os.replace(tmp, _SO)
    return _SO


def _lib():
    global _LIB
    if _LIB is None:
        build()
        L = ctypes.CDLL(_SO)
        i64 = ctypes.c_int64
        L.synth_frames_c.argtypes = [ctypes.c_uint64, i64, ctypes.c_void_p, i64, i64, i64, i64, ctypes.c_int,
                                     ctypes.c_int32, ctypes.c_int, ctypes.c_void_p, ctypes.c_int]
        L.synth_frames_c.restype = ctypes.c_int
        L.synth_max_threads.argtypes = []
        L.synth_max_threads.restype = ctypes.c_int
        _LIB = L
    return _LIB


def max_threads() -> int:
    return int(_lib().synth_max_threads())


def frames_c(seed: int, frame0: int, nframes: int, channels: int, H: int, W: int, kind: str = "uniform",
             value: int = 0, index=None, dtype=np.int32, out: np.ndarray = None, nthreads: int = 0) -> np.ndarray:
    """``frames`` in C with OpenMP.  index: optional sequence of global frame indices (frame n of the result is
    global frame index[n]; default frame0 + n).  dtype int32 or uint8 (kinds whose values fit)."""
    if kind not in KIND_CODE:
        raise ValueError(f"unknown kind {kind!r}; one of {KINDS}")
    dtype = np.dtype(dtype)
    if dtype not in (np.dtype(np.int32), np.dtype(np.uint8)):
        raise TypeError("dtype must be int32 or uint8")
    shape = (nframes, channels, H, W)
    if out is None:
        out = np.empty(shape, dtype=dtype)
    if out.shape != shape or out.dtype != dtype or not out.flags.c_contiguous:
        raise ValueError(f"out must be a C-contiguous {dtype} array of shape {shape}")
    idx = None
    if index is not None:
        idx = np.ascontiguousarray(np.asarray(index, dtype=np.int64))
        if idx.shape != (nframes,):
            raise ValueError("index must hold one global frame index per frame")
    rc = _lib().synth_frames_c(seed & 0xFFFFFFFFFFFFFFFF, frame0, idx.ctypes.data if idx is not None else None,
                               nframes, channels, H, W, KIND_CODE[kind], value, dtype.itemsize, out.ctypes.data,
                               int(nthreads or max_threads()))
    if rc != 0:
        raise ValueError("synth_frames_c rejected its arguments")
    return out
