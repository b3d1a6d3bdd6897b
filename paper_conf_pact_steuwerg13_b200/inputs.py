"""Seeded synthetic inputs shared by the tests, bench.py and the oracle driver.

This module holds NONE of the method's arithmetic: only the counter-based
random generator and the workload recipes (shapes, value distributions) that
DESIGN.md §"Input recipe" states.  Both sides of every parity test (the CUDA
path and the CPU oracle) receive the same arrays from here.

Generator (SURVEY.md §8(d) "Inputs"): element i of stream `seed` is
splitmix64(seed * 2^32 + i); a uniform float in [0,1) is (x >> 40) * 2^-24,
which is exactly representable in fp32.
"""
from __future__ import annotations

import math

import numpy as np

_M = np.uint64(0xFFFFFFFFFFFFFFFF)
_C1 = np.uint64(0x9E3779B97F4A7C15)
_C2 = np.uint64(0xBF58476D1CE4E5B9)
_C3 = np.uint64(0x94D049BB133111EB)

# seeds fixed by BASELINE.md §4
SEED_DOT_A, SEED_DOT_B = 1, 2
SEED_SCAN_I32, SEED_SCAN_F32 = 3, 4
SEED_SOBEL, SEED_GAUSS = 5, 6
SEED_LMOSEM = 7


def splitmix64(seed: int, start: int, count: int) -> np.ndarray:
    """uint64 stream: splitmix64(seed<<32 + i) for i in [start, start+count)."""
    with np.errstate(over="ignore"):
        x = np.arange(start, start + count, dtype=np.uint64) + np.uint64((seed & 0xFFFFFFFF) << 32)
        z = x + _C1
        z = (z ^ (z >> np.uint64(30))) * _C2
        z = (z ^ (z >> np.uint64(27))) * _C3
        z = z ^ (z >> np.uint64(31))
    return z


def uniform_f32(seed: int, n: int, start: int = 0, chunk: int = 1 << 24) -> np.ndarray:
    """U[0,1) fp32 values, exact multiples of 2^-24."""
    out = np.empty(n, dtype=np.float32)
    for a in range(0, n, chunk):
        b = min(n, a + chunk)
        z = splitmix64(seed, start + a, b - a)
        out[a:b] = (z >> np.uint64(40)).astype(np.float32) * np.float32(2.0 ** -24)
    return out


def uniform_int(seed: int, n: int, lo: int, hi: int, dtype=np.int32, start: int = 0,
                chunk: int = 1 << 24) -> np.ndarray:
    """Integers uniform in [lo, hi] (inclusive) via multiply-shift of the top 32 bits."""
    out = np.empty(n, dtype=dtype)
    span = np.uint64(hi - lo + 1)
    for a in range(0, n, chunk):
        b = min(n, a + chunk)
        z = splitmix64(seed, start + a, b - a)
        v = ((z >> np.uint64(32)) * span) >> np.uint64(32)
        out[a:b] = (v.astype(np.int64) + lo).astype(dtype)
    return out


def image_u8(seed: int, rows: int, cols: int) -> np.ndarray:
    """U{0..255} image (Sobel, seed 5)."""
    return uniform_int(seed, rows * cols, 0, 255, np.uint8).reshape(rows, cols)


def image_f32(seed: int, rows: int, cols: int) -> np.ndarray:
    """U[0,1) image (Gaussian, seed 6)."""
    return uniform_f32(seed, rows * cols).reshape(rows, cols)


def mandel_grid(rows: int, cols: int) -> np.ndarray:
    """The Matrix<float2> of pixel coordinates c (reading A22/A23).

    Window [-2, 1) x [-1.125, 1.125): cx = -2 + col*(3/cols), cy = -1.125 +
    row*(2.25/rows).  For cols = 4096, rows = 3072 both steps are 3*2^-12, so
    every c is exact in fp32.  Returns float32 array [rows, cols, 2] (re, im).
    """
    cx = (-2.0 + np.arange(cols, dtype=np.float64) * (3.0 / cols)).astype(np.float32)
    cy = (-1.125 + np.arange(rows, dtype=np.float64) * (2.25 / rows)).astype(np.float32)
    g = np.empty((rows, cols, 2), dtype=np.float32)
    g[:, :, 0] = cx[None, :]
    g[:, :, 1] = cy[:, None]
    return g


def lmosem_events(seed: int, nev: int, N: int, start: int = 0) -> np.ndarray:
    """List-mode events as endpoint pairs (reading A29).

    Each event e uses stream positions 4(start+e)..4(start+e)+3 for
    (theta0, z0, theta1, z1); endpoints lie on the cylinder of radius 0.75 N
    about the axis (N/2, N/2, z): p = (N/2 + R cos theta, N/2 + R sin theta, z),
    theta ~ U[0, 2pi), z ~ U[0, N).  Computed in float64, rounded to float32.
    Returns float32 [nev, 6] = (x0, y0, z0, x1, y1, z1).
    """
    u = uniform_f32(seed, 4 * nev, start=4 * start).astype(np.float64).reshape(nev, 4)
    R = 0.75 * N
    c = N / 2.0
    t0 = 2.0 * math.pi * u[:, 0]
    t1 = 2.0 * math.pi * u[:, 2]
    ev = np.empty((nev, 6), dtype=np.float64)
    ev[:, 0] = c + R * np.cos(t0)
    ev[:, 1] = c + R * np.sin(t0)
    ev[:, 2] = N * u[:, 1]
    ev[:, 3] = c + R * np.cos(t1)
    ev[:, 4] = c + R * np.sin(t1)
    ev[:, 5] = N * u[:, 3]
    return ev.astype(np.float32)

