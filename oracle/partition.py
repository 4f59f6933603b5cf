"""Partition function of the radix join -- TEST INFRASTRUCTURE ONLY.

The paper partitions both inputs "in such a way that elements belonging to
the same output partition" end up together (PAPER.md P579-586, §4.1) over
one or more passes (P531-534, P589-593) but never names the partition
function.  DESIGN.md reading R1 fixes it:

  h(k) = fmix32(k as u32)  for 32-bit keys (MurmurHash3 finaliser)
  h(k) = fmix64(k as u64)  for 64-bit keys (splitmix64 finaliser)
  h(k) = k                 for HAPE_PART_IDENTITY (the equal-size partitions
                           of P802-804 on dense keys)

and the bit fields of h (reading R3):
  destination GPU  = top g = log2(G) bits of h
  pass-1 bucket    = bits [B2, B2+B1)   (bits [0, B1) for a one-pass plan)
  pass-2 bucket    = bits [0, B2)
  partition id     = bits [0, B1+B2), i.e. the final partition
                     q = bucket1 * 2^B2 + bucket2 (pass-1 major)

This module restates those definitions in numpy for the invariant tests; it
shares no code with the CUDA path.  Pinned in tests/test_oracle_pins.py by
the published MurmurHash3_x86_32 vectors (the x86_32 hash of the empty string
with seed s is fmix32(s)) and splitmix64 vectors.
"""
from __future__ import annotations

import numpy as np

_U32 = np.uint32
_U64 = np.uint64


def fmix32(x: np.ndarray) -> np.ndarray:
    h = np.asarray(x).astype(np.int64).astype(np.uint64) & _U64(0xFFFFFFFF)
    h = h.astype(np.uint32)
    with np.errstate(over="ignore"):
        h ^= h >> _U32(16)
        h = (h * _U32(0x85EBCA6B)).astype(np.uint32)
        h ^= h >> _U32(13)
        h = (h * _U32(0xC2B2AE35)).astype(np.uint32)
        h ^= h >> _U32(16)
    return h


def fmix64(x: np.ndarray) -> np.ndarray:
    z = np.asarray(x).astype(np.int64).view(np.uint64).copy()
    with np.errstate(over="ignore"):
        z ^= z >> _U64(30); z *= _U64(0xBF58476D1CE4E5B9)
        z ^= z >> _U64(27); z *= _U64(0x94D049BB133111EB)
        z ^= z >> _U64(31)
    return z


def h(keys: np.ndarray, identity: bool = False) -> np.ndarray:
    """Partition hash as uint64 (32-bit keys give values < 2^32)."""
    keys = np.asarray(keys)
    if identity:
        if keys.dtype == np.int32:
            return keys.view(np.uint32).astype(np.uint64)
        return keys.view(np.uint64)
    if keys.dtype == np.int32:
        return fmix32(keys).astype(np.uint64)
    return fmix64(keys)


def bits(hv: np.ndarray, lo: int, n: int) -> np.ndarray:
    return ((hv >> _U64(lo)) & _U64((1 << n) - 1)).astype(np.int64)


def partition_id(keys: np.ndarray, b1: int, b2: int, identity: bool = False) -> np.ndarray:
    """Final partition q = bucket1 * 2^b2 + bucket2 (pass-1 major order)."""
    hv = h(keys, identity)
    return bits(hv, b2, b1) * (1 << b2) + bits(hv, 0, b2)


def destination(keys: np.ndarray, world: int, identity: bool = False) -> np.ndarray:
    """Owner rank = top log2(world) bits of h (32 or 64 bit word)."""
    if world == 1:
        return np.zeros(len(keys), np.int64)
    g = int(world).bit_length() - 1
    assert (1 << g) == world, "world size must be a power of two"
    keys = np.asarray(keys)
    W = 32 if keys.dtype == np.int32 else 64
    hv = h(keys, identity)
    return (hv >> _U64(W - g)).astype(np.int64)
