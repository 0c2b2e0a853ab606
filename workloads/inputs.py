"""Seeded synthetic input streams ("Inputs").

Counter-based SplitMix64: value k of stream `seed` depends only on (seed, k),
so any slice of a stream can be regenerated independently (both sides read the
same host bytes; nothing here knows what the graph computes).

  f32: (z >> 40) * 2^-23 - 1   -> exactly representable, uniform on [-1, 1)
  i32: (int32)(z >> 32)        -> full-range signed keys
"""
from __future__ import annotations

import numpy as np

_G = np.uint64(0x9E3779B97F4A7C15)
_M1 = np.uint64(0xBF58476D1CE4E5B9)
_M2 = np.uint64(0x94D049BB133111EB)


def splitmix64(seed: int, start: int, count: int) -> np.ndarray:
    idx = np.arange(start, start + count, dtype=np.uint64)
    with np.errstate(over="ignore"):
        z = np.uint64(seed & 0xFFFFFFFFFFFFFFFF) + (idx + np.uint64(1)) * _G
        z = (z ^ (z >> np.uint64(30))) * _M1
        z = (z ^ (z >> np.uint64(27))) * _M2
        z = z ^ (z >> np.uint64(31))
    return z


def uniform_f32(seed: int, count: int, start: int = 0) -> np.ndarray:
    z = splitmix64(seed, start, count)
    return ((z >> np.uint64(40)).astype(np.float64) * 2.0 ** -23 - 1.0).astype(np.float32)


def keys_i32(seed: int, count: int, start: int = 0) -> np.ndarray:
    z = splitmix64(seed, start, count)
    return (z >> np.uint64(32)).astype(np.uint32).view(np.int32)


# Per-config default seeds.
SEEDS = {"fft64": 0xF0F1, "bitonic32": 0xB170, "fmradio10": 0xF3,
         "beamformer12x4": 0xBEA3, "filterbank64": 0xFB64,
         "bitonicrec32": 0xB1C, "dct16": 0xDC7, "matmul16": 0x3A7, "matmul3_16": 0x3A3, "des16": 0xDE5, "echo64": 0xEC0}


def make_input(dtype: str, count: int, seed: int, variant: str = "uniform", block: int = 32) -> np.ndarray:
    """Input stream of `count` items.  Variants exercise edge cases:

    uniform   - the default distribution for the dtype
    ties      - i32 keys mod 8 (many equal keys)
    sorted    - i32 blocks of `block` keys already ascending
    reversed  - i32 blocks of `block` keys descending
    impulse   - f32 delta at complex index 1 of every 2*block-float FFT row
    dc        - f32 all-ones real part
    smallint  - f32 integers in [-3, 3] (exact-arithmetic pins)
    fmtone    - f32 FM tone cos(2*pi*0.1 t + 5 sin(2*pi*0.001 t))
    """
    if dtype == "i32":
        x = keys_i32(seed, count)
        if variant == "ties":
            x = (x % 8).astype(np.int32)
        elif variant in ("sorted", "reversed"):
            n = count - count % block
            y = np.sort(x[:n].reshape(-1, block), axis=1)
            if variant == "reversed":
                y = y[:, ::-1]
            x = np.concatenate([y.reshape(-1), x[n:]]).astype(np.int32)
        return np.ascontiguousarray(x, dtype=np.int32)
    if variant == "uniform":
        return uniform_f32(seed, count)
    if variant == "smallint":
        z = splitmix64(seed, 0, count)
        return ((z >> np.uint64(33)) % np.uint64(7)).astype(np.float32) - 3.0
    if variant == "impulse":
        x = np.zeros(count, np.float32)
        row = 2 * block
        x[2::row] = 1.0
        return x
    if variant == "dc":
        x = np.zeros(count, np.float32)
        x[0::2] = 1.0
        return x
    if variant == "fmtone":
        t = np.arange(count, dtype=np.float64)
        return np.cos(2 * np.pi * 0.1 * t + 5 * np.sin(2 * np.pi * 0.001 * t)).astype(np.float32)
    raise ValueError(variant)
