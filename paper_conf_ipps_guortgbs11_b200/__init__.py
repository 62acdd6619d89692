"""B200-native ArrayOL downscaler (Guo et al., HIPS 2011) -- Python binding.

Thin marshalling over the C ABI of ``include/aol.h`` (``libaol.so``): every
step of the path runs in the library's sm_100a kernels; PyTorch only supplies
device memory and the current CUDA stream.  There is no CPU fallback -- if the
extension is missing, importing an entry point raises.

Paper citations: tiler semantics Section IV
(P:L292-319), SaC tiler functions Fig. 4-7, the downscaler
tilers Fig. 10, the task Fig. 5.
"""
from __future__ import annotations

import ctypes
from typing import Optional, Sequence

import torch

from . import _lib
from ._lib import FLAGS  # noqa: F401  (launch-option flag bits, include/aol.h AOL_FLAG_*)
from ._lib import RGB8  # noqa: F401
from ._lib import (FILTER_H, FILTER_V, AolError, I16, I32, I64, PRESET_H_IN, PRESET_H_OUT, PRESET_V_IN,
                   PRESET_V_OUT, RAW8, RAW16, RAW32, RAW64, SCATTER_FAST, SCATTER_SEQUENTIAL, U8, aol_filter_t,
                   aol_launch_opts_t, aol_plan_t, aol_tiler_t, check, lib)

__all__ = [
    "AolError", "version", "make_tiler", "tiler_preset", "tiler_validate", "tiler_is_injective",
    "tiler_gather", "tiler_scatter", "tiler_scatter_workspace_bytes", "downscale_h", "downscale_v", "downscale_frame", "downscale_frame_plan",
    "frame_checksum", "downscale_frame_host", "FramePlan", "synth_frames", "library_path", "downscale_frame_packed",
    "PRESET_H_IN", "PRESET_H_OUT", "PRESET_V_IN", "PRESET_V_OUT", "SYNTH_KINDS",
    "make_filter", "filter_preset", "filter_validate", "filter_apply", "filter_chain_apply", "last_kernel", "FILTER_H", "FILTER_V", "FLAGS",
]

SYNTH_KINDS = {"uniform": 0, "dark": 1, "signed": 2, "ramp": 3, "constant": 4}
library_path = _lib.LIB_PATH

_TYPED = {torch.uint8: U8, torch.int16: I16, torch.int32: I32, torch.int64: I64}
_RAW = {1: RAW8, 2: RAW16, 4: RAW32, 8: RAW64}


def _dtype_code(t: torch.Tensor) -> int:
    if t.dtype in _TYPED:
        return _TYPED[t.dtype]
    es = t.element_size()
    if es not in _RAW:
        raise TypeError(f"unsupported element size {es}")
    return _RAW[es]


def _stream(stream: Optional[torch.cuda.Stream], device=None) -> ctypes.c_void_p:
    """The given stream, else the current stream of `device` (the tensors' device, not the current one)."""
    s = stream if stream is not None else torch.cuda.current_stream(device)
    return ctypes.c_void_p(s.cuda_stream)


def _out(t: torch.Tensor, shape, dtype, device, name: str) -> torch.Tensor:
    """Check a caller-supplied output: the kernels write exactly `shape` elements of `dtype` on `device`."""
    if tuple(t.shape) != tuple(shape) or t.dtype != dtype or t.device != device:
        raise ValueError(f"{name} must be {dtype} {tuple(shape)} on {device}; got {t.dtype} {tuple(t.shape)} on "
                         f"{t.device}")
    return t


def _checksum_buf(cs: torch.Tensor, n: int, device) -> torch.Tensor:
    if cs.dtype not in (torch.uint64, torch.int64) or cs.numel() < n or cs.device != device:
        raise ValueError(f"checksums must be a uint64/int64 tensor of >= {n} elements on {device}")
    return cs


def _dev(t: torch.Tensor, name: str) -> ctypes.c_void_p:
    if not isinstance(t, torch.Tensor) or not t.is_cuda:
        raise ValueError(f"{name} must be a CUDA tensor")
    if not t.is_contiguous():
        raise ValueError(f"{name} must be contiguous")
    return ctypes.c_void_p(t.data_ptr())


def version() -> int:
    return int(lib().aol_version())


def last_kernel() -> str:
    """Name of the last kernel a library call launched on this thread (aol_debug_last_kernel)."""
    return lib().aol_debug_last_kernel().decode()


# ------------------------------------------------------------------ tilers

def make_tiler(array_shape: Sequence[int], rep_shape: Sequence[int], pattern_shape: Sequence[int],
               origin: Optional[Sequence[int]] = None, paving=None, fitting=None) -> aol_tiler_t:
    """ArrayOL tiler (Fig. 10 record): paving is [array_rank][rep_rank], fitting [array_rank][pattern_rank]."""
    t = aol_tiler_t()
    t.array_rank, t.rep_rank, t.pattern_rank = len(array_shape), len(rep_shape), len(pattern_shape)
    for k, v in enumerate(array_shape):
        t.array_shape[k] = int(v)
    for k, v in enumerate(rep_shape):
        t.rep_shape[k] = int(v)
    for k, v in enumerate(pattern_shape):
        t.pattern_shape[k] = int(v)
    for a in range(len(array_shape)):
        t.origin[a] = int(origin[a]) if origin is not None else 0
        for j in range(len(rep_shape)):
            t.paving[a][j] = int(paving[a][j]) if paving is not None else 0
        for k in range(len(pattern_shape)):
            t.fitting[a][k] = int(fitting[a][k]) if fitting is not None else 0
    return t


def _shapes(t: aol_tiler_t):
    return (tuple(t.array_shape[k] for k in range(t.array_rank)),
            tuple(t.rep_shape[k] for k in range(t.rep_rank)),
            tuple(t.pattern_shape[k] for k in range(t.pattern_rank)))


def tiler_preset(which: int, H: int, W: int) -> aol_tiler_t:
    t = aol_tiler_t()
    check(lib().aol_tiler_preset(which, H, W, ctypes.byref(t)))
    return t


def tiler_validate(t: aol_tiler_t) -> None:
    check(lib().aol_tiler_validate(ctypes.byref(t)))


def tiler_is_injective(t: aol_tiler_t) -> bool:
    v = ctypes.c_int(0)
    check(lib().aol_tiler_is_injective(ctypes.byref(t), ctypes.byref(v)))
    return bool(v.value)


def tiler_scatter_workspace_bytes(t: aol_tiler_t) -> int:
    """Device workspace bytes a SEQUENTIAL scatter with tiler t needs (0 if none)."""
    return int(lib().aol_tiler_scatter_workspace_bytes(ctypes.byref(t)))


def tiler_gather(t: aol_tiler_t, array: torch.Tensor, out: Optional[torch.Tensor] = None,
                 stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """tiles[r][i] = array[(o + P.r + F.i) mod s]  (Fig. 4); returns [rep..., pattern...]."""
    arr, rep, pat = _shapes(t)
    if tuple(array.shape) != arr:
        raise ValueError(f"array shape {tuple(array.shape)} != tiler array shape {arr}")
    if out is None:
        out = torch.empty(rep + pat, dtype=array.dtype, device=array.device)
    _out(out, rep + pat, array.dtype, array.device, "out")
    with torch.cuda.device(array.device):
        check(lib().aol_tiler_gather(ctypes.byref(t), _dtype_code(array), _dev(array, "array"), _dev(out, "out"),
                                     _stream(stream, array.device)))
    return out


def tiler_scatter(t: aol_tiler_t, tiles: torch.Tensor, array: torch.Tensor, mode: str = "fast",
                  workspace: Optional[torch.Tensor] = None, stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """array[(o + P.r + F.i) mod s] = tiles[r][i] in place (Fig. 6).  mode: 'fast' | 'sequential'."""
    arr, rep, pat = _shapes(t)
    if tuple(array.shape) != arr:
        raise ValueError(f"array shape {tuple(array.shape)} != tiler array shape {arr}")
    _out(tiles, rep + pat, array.dtype, array.device, "tiles")
    m = {"fast": SCATTER_FAST, "sequential": SCATTER_SEQUENTIAL}[mode]
    ws_ptr, ws_bytes = ctypes.c_void_p(0), 0
    need = int(lib().aol_tiler_scatter_workspace_bytes(ctypes.byref(t))) if m == SCATTER_SEQUENTIAL else 0
    if need > 0:   # 0: the library proved the tiler injective (no claims needed) or the mode is FAST
        if workspace is None:
            workspace = torch.empty(need, dtype=torch.uint8, device=array.device)
        if workspace.device != array.device:
            raise ValueError("workspace must be on the array's device")
        ws_ptr, ws_bytes = _dev(workspace, "workspace"), workspace.numel() * workspace.element_size()
    with torch.cuda.device(array.device):
        check(lib().aol_tiler_scatter(ctypes.byref(t), _dtype_code(array), _dev(tiles, "tiles"),
                                      _dev(array, "array"), m, ws_ptr, ws_bytes, _stream(stream, array.device)))
    return array


# ------------------------------------------------- generic repetition (f3)

def make_filter(tin: aol_tiler_t, tout: aol_tiler_t, window_start: Sequence[int], window_len: int,
                divisor: int) -> aol_filter_t:
    """A run-time ArrayOL repetition: gather with tin, windowed-sum task, scatter with tout."""
    f = aol_filter_t()
    f.in_, f.out = tin, tout
    f.n_windows = len(window_start)
    f.window_len, f.divisor = int(window_len), int(divisor)
    for k, v in enumerate(window_start):
        f.window_start[k] = int(v)
    return f


def filter_preset(kind: int, planes: int, H: int, W: int) -> aol_filter_t:
    f = aol_filter_t()
    check(lib().aol_filter_preset(kind, planes, H, W, ctypes.byref(f)))
    return f


def filter_validate(f: aol_filter_t) -> None:
    check(lib().aol_filter_validate(ctypes.byref(f)))


def filter_apply(f: aol_filter_t, x: torch.Tensor, out: Optional[torch.Tensor] = None,
                 stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """Run the fused generic repetition: x int32 shaped f.in_ array -> out int32 shaped f.out array."""
    a_in, _, _ = _shapes(f.in_)
    a_out, _, _ = _shapes(f.out)
    if x.dtype != torch.int32 or tuple(x.shape) != a_in:
        raise ValueError(f"x must be int32 {a_in}")
    if out is None:
        out = torch.zeros(a_out, dtype=torch.int32, device=x.device)
    _out(out, a_out, torch.int32, x.device, "out")
    with torch.cuda.device(x.device):
        check(lib().aol_filter_apply(ctypes.byref(f), _dev(x, "x"), _dev(out, "out"), _stream(stream, x.device)))
    return out


def filter_chain_apply(f1: aol_filter_t, f2: aol_filter_t, x: torch.Tensor, out: Optional[torch.Tensor] = None,
                       workspace: Optional[torch.Tensor] = None,
                       stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """out = f2(f1(x)) in one fused kernel (the intermediate array never stored) when the chain qualifies,
    else two launches through `workspace` (int32 tensor of f1's output array, or None -> error naming why)."""
    a_in, _, _ = _shapes(f1.in_)
    a_out, _, _ = _shapes(f2.out)
    if x.dtype != torch.int32 or tuple(x.shape) != a_in:
        raise ValueError(f"x must be int32 {a_in}")
    if out is None:
        out = torch.zeros(a_out, dtype=torch.int32, device=x.device)
    _out(out, a_out, torch.int32, x.device, "out")
    wp, wb = ctypes.c_void_p(0), 0
    if workspace is not None:
        wp, wb = _dev(workspace, "workspace"), workspace.numel() * workspace.element_size()
    with torch.cuda.device(x.device):
        check(lib().aol_filter_chain_apply(ctypes.byref(f1), ctypes.byref(f2), _dev(x, "x"), _dev(out, "out"), wp, wb,
                                           _stream(stream, x.device)))
    return out


# ------------------------------------------------------------------ filters

def _planes(x: torch.Tensor):
    if x.dim() < 2:
        raise ValueError("expected [..., H, W]")
    H, W = x.shape[-2:]
    planes = 1
    for d in x.shape[:-2]:
        planes *= d
    return planes, H, W


def downscale_h(x: torch.Tensor, out: Optional[torch.Tensor] = None,
                stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """Horizontal filter: int32 [..., H, W] -> [..., H, 3W/8]."""
    if x.dtype != torch.int32:
        raise TypeError("downscale_h takes int32")
    planes, H, W = _planes(x)
    if out is None:
        out = torch.empty(x.shape[:-1] + (3 * (W // 8),), dtype=torch.int32, device=x.device)
    _out(out, x.shape[:-1] + (3 * (W // 8),), torch.int32, x.device, "out")
    with torch.cuda.device(x.device):
        check(lib().aol_downscale_h(_dev(x, "x"), _dev(out, "out"), planes, H, W, _stream(stream, x.device)))
    return out


def downscale_v(y: torch.Tensor, out: Optional[torch.Tensor] = None,
                stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """Vertical filter: int32 [..., H, W] -> [..., 4H/9, W]."""
    if y.dtype != torch.int32:
        raise TypeError("downscale_v takes int32")
    planes, H, W = _planes(y)
    if out is None:
        out = torch.empty(y.shape[:-2] + (4 * (H // 9), W), dtype=torch.int32, device=y.device)
    _out(out, y.shape[:-2] + (4 * (H // 9), W), torch.int32, y.device, "out")
    with torch.cuda.device(y.device):
        check(lib().aol_downscale_v(_dev(y, "y"), _dev(out, "out"), planes, H, W, _stream(stream, y.device)))
    return out


def _opts(opts) -> Optional[aol_launch_opts_t]:
    if opts is None:
        return None
    o = aol_launch_opts_t()
    for k, v in dict(opts).items():
        setattr(o, k, int(v))
    return o


def downscale_frame(x: torch.Tensor, out: Optional[torch.Tensor] = None, checksums=None, opts=None,
                    stream: Optional[torch.cuda.Stream] = None, out_dtype: Optional[torch.dtype] = None):
    """Fused downscaler: x [frames][channels][H][W] (int32 or uint8) -> [frames][channels][4H/9][3W/8]
    int32, or int16 (out_dtype=torch.int16, uint8 input only: outputs lie in [-5, 255]).

    checksums: None (skip), True (allocate), or a uint64/int64 CUDA tensor [frames].
    Returns (out, checksums_or_None)."""
    if x.dim() != 4:
        raise ValueError("x must be [frames][channels][H][W]")
    if x.dtype not in (torch.int32, torch.uint8):
        raise TypeError("x must be int32 or uint8")
    N, C, H, W = x.shape
    odt = out.dtype if out is not None else (out_dtype or torch.int32)
    if odt not in (torch.int32, torch.int16):
        raise TypeError("output must be int32 or int16")
    if out is None:
        out = torch.empty((N, C, 4 * (H // 9), 3 * (W // 8)), dtype=odt, device=x.device)
    _out(out, (N, C, 4 * (H // 9), 3 * (W // 8)), odt, x.device, "out")
    cs = checksums
    if cs is True:
        cs = torch.empty(N, dtype=torch.uint64, device=x.device)
    cs_ptr = _dev(_checksum_buf(cs, N, x.device), "checksums") if cs is not None else ctypes.c_void_p(0)
    o = _opts(opts)
    with torch.cuda.device(x.device):
        check(lib().aol_downscale_frame_out(_dev(x, "x"), _TYPED[x.dtype], _dev(out, "out"), _TYPED[odt], N, C, H, W,
                                            cs_ptr, ctypes.byref(o) if o is not None else None,
                                            _stream(stream, x.device)))
    return out, cs


def downscale_frame_packed(x: torch.Tensor, out: Optional[torch.Tensor] = None, checksums=None, opts=None,
                           stream: Optional[torch.cuda.Stream] = None, out_dtype: Optional[torch.dtype] = None):
    """Fused downscaler on packed 24-bit pixels (OpenCV's interleaved frames): x uint8
    [frames][H][W][3] -> planar [frames][3][4H/9][3W/8] int32 (or int16 with out_dtype=torch.int16).
    Same integers and checksums as downscale_frame on the planar frames x.permute(0, 3, 1, 2)."""
    if x.dim() != 4 or x.shape[3] != 3 or x.dtype != torch.uint8:
        raise ValueError("x must be uint8 [frames][H][W][3]")
    N, H, W, _ = x.shape
    odt = out.dtype if out is not None else (out_dtype or torch.int32)
    if odt not in (torch.int32, torch.int16):
        raise TypeError("output must be int32 or int16")
    if out is None:
        out = torch.empty((N, 3, 4 * (H // 9), 3 * (W // 8)), dtype=odt, device=x.device)
    _out(out, (N, 3, 4 * (H // 9), 3 * (W // 8)), odt, x.device, "out")
    cs = checksums
    if cs is True:
        cs = torch.empty(N, dtype=torch.uint64, device=x.device)
    cs_ptr = _dev(_checksum_buf(cs, N, x.device), "checksums") if cs is not None else ctypes.c_void_p(0)
    o = _opts(opts)
    with torch.cuda.device(x.device):
        check(lib().aol_downscale_frame_out(_dev(x, "x"), RGB8, _dev(out, "out"), _TYPED[odt], N, 3, H, W, cs_ptr,
                                            ctypes.byref(o) if o is not None else None, _stream(stream, x.device)))
    return out, cs


class FramePlan:
    """A persistent launch plan (aol_frame_plan_*): the fused downscale of fixed tensors x -> out resolved once;
    launch() is then one kernel launch (the d1 single-frame case).  x: planar int32/uint8 [N][C][H][W], or
    packed uint8 [N][H][W][3] with packed=True.  Keep x / out / checksums alive while the plan is used;
    launches of one plan must be stream-ordered."""

    def __init__(self, x: torch.Tensor, out: Optional[torch.Tensor] = None, checksums=None, opts=None,
                 out_dtype: Optional[torch.dtype] = None, packed: bool = False, stream=None):
        if packed:
            if x.dim() != 4 or x.shape[3] != 3 or x.dtype != torch.uint8:
                raise ValueError("packed x must be uint8 [frames][H][W][3]")
            N, H, W, C = x.shape
            code = RGB8
        else:
            if x.dim() != 4 or x.dtype not in (torch.int32, torch.uint8):
                raise ValueError("x must be int32 or uint8 [frames][channels][H][W]")
            N, C, H, W = x.shape
            code = _TYPED[x.dtype]
        odt = out.dtype if out is not None else (out_dtype or torch.int32)
        if out is None:
            out = torch.empty((N, C, 4 * (H // 9), 3 * (W // 8)), dtype=odt, device=x.device)
        _out(out, (N, C, 4 * (H // 9), 3 * (W // 8)), odt, x.device, "out")
        if checksums is True:
            checksums = torch.empty(N, dtype=torch.uint64, device=x.device)
        self.x, self.out, self.checksums = x, out, checksums
        self._cs = (_dev(_checksum_buf(checksums, N, x.device), "checksums") if checksums is not None
                    else ctypes.c_void_p(0))
        self._h = ctypes.c_void_p(0)
        o = _opts(opts)
        self._lib = lib()
        with torch.cuda.device(x.device):
            check(self._lib.aol_frame_plan_create(_dev(x, "x"), code, _dev(out, "out"), _TYPED[odt], N, C, H, W,
                                                  ctypes.byref(o) if o is not None else None, ctypes.byref(self._h)))
        self._stream = _stream(stream, x.device)
        self._launch = self._lib.aol_frame_plan_launch

    def launch(self):
        """Enqueue one downscale on the plan's stream (the current stream at creation unless given)."""
        st = self._launch(self._h, self._cs, self._stream)
        if st:
            check(st)
        return self.out, self.checksums

    def info(self) -> dict:
        p = aol_plan_t()
        check(self._lib.aol_frame_plan_info(self._h, ctypes.byref(p)))
        return {f: getattr(p, f) for f, _ in aol_plan_t._fields_}

    def close(self):
        if self._h:
            check(self._lib.aol_frame_plan_destroy(self._h))
            self._h = ctypes.c_void_p(0)

    def __del__(self):
        try:
            if self._h:
                self._lib.aol_frame_plan_destroy(self._h)
        except Exception:
            pass


def downscale_frame_plan(frames: int, channels: int, H: int, W: int, dtype=torch.int32, opts=None,
                         out_dtype=torch.int32) -> dict:
    """dtype: torch.int32 / torch.uint8 planes, or "rgb8" for packed 24-bit pixels."""
    p = aol_plan_t()
    o = _opts(opts)
    code = RGB8 if dtype == "rgb8" else _TYPED[dtype]
    check(lib().aol_downscale_frame_plan_out(code, _TYPED[out_dtype], frames, channels, H, W,
                                             ctypes.byref(o) if o is not None else None, ctypes.byref(p)))
    return {f: getattr(p, f) for f, _ in aol_plan_t._fields_}


def frame_checksum(z: torch.Tensor, out: Optional[torch.Tensor] = None,
                   stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """Per-frame checksum of an int32 [frames][channels][Ho][Wo] batch."""
    if z.dim() != 4 or z.dtype != torch.int32:
        raise ValueError("z must be int32 [frames][channels][Ho][Wo]")
    N, C, Ho, Wo = z.shape
    if out is None:
        out = torch.empty(N, dtype=torch.uint64, device=z.device)
    _checksum_buf(out, N, z.device)
    with torch.cuda.device(z.device):
        check(lib().aol_frame_checksum(_dev(z, "z"), N, C, Ho, Wo, _dev(out, "out"), _stream(stream, z.device)))
    return out


def host_workspace_bytes(chunk_frames: int, channels: int, H: int, W: int, dtype=torch.int32) -> int:
    return int(lib().aol_downscale_frame_host_workspace_bytes(_TYPED[dtype], chunk_frames, channels, H, W))


def downscale_frame_host(x: torch.Tensor, out: Optional[torch.Tensor] = None, checksums: bool = True,
                         chunk_frames: int = 16, workspace: Optional[torch.Tensor] = None, streams=None,
                         device=None, packed: bool = False):
    """End-to-end from HOST memory (pinned for overlap): H2D, fused kernel, D2H, pipelined.
    x: planar [N][C][H][W] int32 / uint8, or with packed=True uint8 [N][H][W][3] 24-bit pixels.
    Blocking.  Returns (out_host, checksums_host_or_None)."""
    if x.is_cuda:
        raise ValueError("x must be a host tensor")
    if not x.is_contiguous():
        raise ValueError("x must be contiguous")
    if packed:
        if x.dim() != 4 or x.shape[3] != 3 or x.dtype != torch.uint8:
            raise ValueError("packed x must be uint8 [frames][H][W][3]")
        N, H, W, C = x.shape
    else:
        N, C, H, W = x.shape
    device = torch.device(device if device is not None else "cuda")
    if out is None:
        out = torch.empty((N, C, 4 * (H // 9), 3 * (W // 8)), dtype=torch.int32, pin_memory=x.is_pinned())
    _out(out, (N, C, 4 * (H // 9), 3 * (W // 8)), torch.int32, torch.device("cpu"), "out")
    if not out.is_contiguous():
        raise ValueError("out must be contiguous")
    cs = torch.empty(N, dtype=torch.uint64, pin_memory=x.is_pinned()) if checksums else None
    chunk = max(1, min(chunk_frames, N))
    code = RGB8 if packed else _TYPED[x.dtype]
    need = int(lib().aol_downscale_frame_host_workspace_bytes(code, chunk, C, H, W))
    if workspace is None:
        workspace = torch.empty(need, dtype=torch.uint8, device=device)
    if streams is None:
        streams = [torch.cuda.Stream(device=device) for _ in range(3)]
    sp = [ctypes.c_void_p(s.cuda_stream) for s in streams]
    with torch.cuda.device(workspace.device):
        check(lib().aol_downscale_frame_host(
            ctypes.c_void_p(x.data_ptr()), code, ctypes.c_void_p(out.data_ptr()), N, C, H, W,
            ctypes.c_void_p(cs.data_ptr()) if cs is not None else ctypes.c_void_p(0), chunk,
            _dev(workspace, "workspace"), workspace.numel() * workspace.element_size(), sp[0], sp[1], sp[2]))
    return out, cs


def synth_frames(seed: int, frame0: int, nframes: int, channels: int, H: int, W: int, kind: str = "uniform",
                 value: int = 0, dtype=torch.int32, device=None, out: Optional[torch.Tensor] = None,
                 stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
    """Synthetic frames on the device (same counter-based generator as synth/)."""
    if out is None:
        out = torch.empty((nframes, channels, H, W), dtype=dtype,
                          device=device if device is not None else "cuda")
    if out.numel() != nframes * channels * H * W or out.dtype not in (torch.int32, torch.uint8):
        raise ValueError(f"out must hold {nframes}x{channels}x{H}x{W} int32 or uint8 elements")
    with torch.cuda.device(out.device):
        check(lib().aol_synth_frames(seed & 0xFFFFFFFFFFFFFFFF, frame0, nframes, channels, H, W, SYNTH_KINDS[kind],
                                     value, _TYPED[out.dtype], _dev(out, "out"), _stream(stream, out.device)))
    return out
