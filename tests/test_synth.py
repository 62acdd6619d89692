"""The seeded input generator (synth/) -- infrastructure shared by both sides."""
import numpy as np

import synth


def test_splitmix64_reference_values():
    """SplitMix64 (Steele, Lea, Flood 2014) seeded with 0 produces 0xE220A8397B1DCDAF,
    then 0x6E789E6AA1B965F4 (the published first outputs)."""
    z = synth.splitmix64(np.array([0, 0x9E3779B97F4A7C15], dtype=np.uint64))
    assert int(z[0]) == 0xE220A8397B1DCDAF
    assert int(z[1]) == 0x6E789E6AA1B965F4


def test_frames_counter_based():
    a = synth.frames(5, 0, 4, 3, 9, 16)
    b = synth.frames(5, 2, 2, 3, 9, 16)
    assert np.array_equal(a[2:], b)
    assert not np.array_equal(a[0], a[1])
    assert not np.array_equal(synth.frames(6, 0, 1, 3, 9, 16), a[:1])


def test_ranges():
    u = synth.frames(1, 0, 2, 3, 18, 64, "uniform")
    assert u.min() >= 0 and u.max() <= 255 and u.max() > 200
    d = synth.frames(1, 0, 2, 3, 18, 64, "dark")
    assert d.min() >= 0 and d.max() <= 7
    s = synth.frames(1, 0, 2, 3, 18, 64, "signed")
    assert s.min() >= -(1 << 26) and s.max() < (1 << 26) and s.min() < 0
    r = synth.frames(1, 0, 1, 2, 3, 40, "ramp")
    assert np.array_equal(r[0, 1, 2], np.arange(40))
    c = synth.frames(1, 0, 1, 1, 2, 8, "constant", value=-9)
    assert np.all(c == -9)


def test_c_generator_equals_numpy():
    """synth.c (OpenMP, used for bench-size oracle inputs) produces the numpy generator's frames bit for bit,
    for every kind, both element types, a seed above 2^63 and an explicit global-frame index list."""
    for kind in synth.KINDS:
        for seed in (0, 7, (1 << 64) - 3):
            a = synth.frames(seed, 3, 2, 3, 9, 24, kind, value=-5)
            b = synth.frames_c(seed, 3, 2, 3, 9, 24, kind, value=-5)
            assert np.array_equal(a, b), (kind, seed)
    u = synth.frames_c(11, 0, 2, 3, 9, 32, "uniform", dtype=np.uint8)
    assert u.dtype == np.uint8 and np.array_equal(u.astype(np.int32), synth.frames(11, 0, 2, 3, 9, 32))
    idx = [5, 0, 257, 5]
    c = synth.frames_c(2, 0, 4, 3, 9, 16, index=idx)
    for n, g in enumerate(idx):
        assert np.array_equal(c[n], synth.frames(2, g, 1, 3, 9, 16)[0])
