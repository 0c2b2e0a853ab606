"""Pins for the oracle on DES (Fig. 4.2a: "compute-intensive applications
such as DES").  The graph (workloads/apps.py des()) is a bit-per-item stream program:
INTO_BITS, IP, 16 Feistel rounds of PERMUTE / XOR_CONST / SBOX split-join / PERMUTE / XOR, IP^-1,
BITS_TO_INT.  Pinned against values the standard fixes, not against the oracle's own tables:

  known answers   six published (key, plaintext, ciphertext) triples, tests/golden/des_kat.json
  involution      decryption (reversed round keys through the same graph) inverts encryption
  complementation E_{~k}(~p) = ~E_k(p) (a structural property of DES: a dropped or misplaced XOR breaks it)
  weak key        with k = 0101010101010101 every round key is zero, so E_k(E_k(p)) = p
  bit kinds       INTO_BITS / BITS_TO_INT against numpy bit unpacking; PERMUTE against fancy indexing;
                  XOR / XOR_CONST against numpy bitwise_xor; a one-SBOX graph on all 64 inputs against the
                  FIPS row/column rule written as a different formula (bit arithmetic on the 6-bit value)
"""
import json
import os

import numpy as np
import pytest

from workloads import apps, inputs
from workloads.spec import Filter, Pipeline, Program, SplitJoin

GOLD = os.path.join(os.path.dirname(__file__), "golden", "des_kat.json")


def blocks_to_words(blocks):
    w = []
    for b in blocks:
        w += [b >> 32, b & 0xFFFFFFFF]
    return np.array(w, dtype=np.uint32).view(np.int32)


def words_to_blocks(y):
    u = y.view(np.uint32)
    return [(int(u[2 * i]) << 32) | int(u[2 * i + 1]) for i in range(len(u) // 2)]


def des_run(oracle_lib, key, blocks, decrypt=False, rounds=16):
    prog = apps.des(rounds, key, decrypt)
    return words_to_blocks(oracle_lib.run(prog, blocks_to_words(blocks), len(blocks)))


def test_des_known_answers(oracle_lib):
    with open(GOLD) as f:
        vec = json.load(f)["vectors"]
    for v in vec:
        k, p, c = (int(v[s], 16) for s in ("key", "plaintext", "ciphertext"))
        assert des_run(oracle_lib, k, [p]) == [c], v["cite"]
        assert des_run(oracle_lib, k, [c], decrypt=True) == [p], v["cite"]


def random_blocks(seed, n):
    w = inputs.keys_i32(seed, 2 * n).view(np.uint32)
    return [(int(w[2 * i]) << 32) | int(w[2 * i + 1]) for i in range(n)]


@pytest.mark.parametrize("key", [0x133457799BBCDFF1, 0xFEDCBA9876543210, 0x0E329232EA6D0D73])
def test_des_decrypt_inverts_encrypt(oracle_lib, key):
    p = random_blocks(5, 64)
    c = des_run(oracle_lib, key, p)
    assert c != p
    assert des_run(oracle_lib, key, c, decrypt=True) == p


def test_des_complementation(oracle_lib):
    M = (1 << 64) - 1
    key = 0x3B3898371520F75E
    p = random_blocks(6, 32)
    c = des_run(oracle_lib, key, p)
    cc = des_run(oracle_lib, key ^ M, [b ^ M for b in p])
    assert cc == [b ^ M for b in c]


def test_des_weak_key_involution(oracle_lib):
    key = 0x0101010101010101
    assert all(sum(k) == 0 for k in apps.des_round_keys(key))
    p = random_blocks(7, 32)
    assert des_run(oracle_lib, key, des_run(oracle_lib, key, p)) == p


def test_des_rates(oracle_lib):
    r = oracle_lib.rates(apps.des(16))
    assert r["in_per_iter"] == 2 and r["out_per_iter"] == 2
    cnt = apps.des(16).count_nodes()
    assert cnt["filters"] == 5 + 16 * 15 and cnt["splitters"] == 16 * 3


def test_bits_roundtrip(oracle_lib):
    x = inputs.keys_i32(9, 40)
    bits = Program("b", "i32", Pipeline([Filter("INTO_BITS")]))
    y = oracle_lib.run(bits, x, 40)
    ref = np.unpackbits(x.astype(">i4").view(np.uint8)).astype(np.int32)   # big-endian: MSB first
    assert np.array_equal(y, ref)
    back = Program("bb", "i32", Pipeline([Filter("INTO_BITS"), Filter("BITS_TO_INT")]))
    assert np.array_equal(oracle_lib.run(back, x, 40), x)


def test_permute_xor_kinds(oracle_lib):
    rng = np.random.default_rng(3)
    idx = rng.integers(0, 7, size=11)
    prog = Program("p", "i32", Pipeline([Filter("PERMUTE", [7] + idx.tolist())]))
    x = inputs.keys_i32(10, 7 * 30)
    assert np.array_equal(oracle_lib.run(prog, x, 30).reshape(30, 11), x.reshape(30, 7)[:, idx])
    prog = Program("x", "i32", Pipeline([Filter("XOR", [5])]))
    x = inputs.keys_i32(11, 10 * 30)
    xr = x.reshape(30, 10)
    assert np.array_equal(oracle_lib.run(prog, x, 30).reshape(30, 5), np.bitwise_xor(xr[:, :5], xr[:, 5:]))
    k = inputs.keys_i32(12, 6)
    prog = Program("xc", "i32", Pipeline([Filter("XOR_CONST", [6] + k.tolist())]))
    x = inputs.keys_i32(13, 6 * 30)
    assert np.array_equal(oracle_lib.run(prog, x, 30).reshape(30, 6), np.bitwise_xor(x.reshape(30, 6), k))


@pytest.mark.parametrize("j", range(8))
def test_sbox_all_inputs(oracle_lib, j):
    prog = Program("s", "i32", Pipeline([Filter("SBOX", apps.DES_S[j])]))
    v = np.arange(64)
    x = ((v[:, None] >> (5 - np.arange(6))[None, :]) & 1).astype(np.int32).ravel()   # b1 = bit 5 of v
    y = oracle_lib.run(prog, x, 64).reshape(64, 4)
    row = ((v >> 4) & 2) | (v & 1)            # outer bits b1 b6
    col = (v >> 1) & 15                        # inner bits b2..b5
    val = np.array(apps.DES_S[j]).reshape(4, 16)[row, col]
    assert np.array_equal(y, ((val[:, None] >> (3 - np.arange(4))[None, :]) & 1))
