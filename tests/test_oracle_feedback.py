"""Pins for the oracle's feedback loops (streams are composed with "pipeline,
split-join, and feedback loop").  StreamIt form: joiner RR(a, b) of the outer input
and the loop stream, body, splitter (duplicate or RR(c, d)) to the output and the loop stream; the
enqueued items are the initial contents of the loop's returning edge.  Pinned against closed forms:

  running sum     ADD(2) body, identity loop, one enqueued 0     -> numpy cumsum (int32, wrapping)
  running max     COMPARE_EXCHANGE body, RR(1,1) split           -> min(x_n, max(x_0..x_{n-1}))
  echo / IIR      y_n = x_n + a y_{n-d} (d enqueued zeros)       -> scipy.signal.lfilter in double
  multirate body  join RR(2,1), FIR(3 taps, pop 3)                -> lfilter of the decimated FIR
  rates           balance holds around the cycle; a rate-inconsistent loop is rejected
  determinism     two schedules x three chunk sizes give the same bytes
"""
import numpy as np
import pytest
import scipy.signal

from workloads import inputs
from workloads.spec import FeedbackLoop, Filter, Pipeline, Program


def running_sum():
    return Program("rsum", "i32", Pipeline([FeedbackLoop(Filter("ADD", [2]), Filter("IDENTITY"), [1, 1], "dup",
                                                         enqueue=[0])]))


def running_max_lag():
    return Program("rmax", "i32", Pipeline([FeedbackLoop(Filter("COMPARE_EXCHANGE", [1]), Filter("IDENTITY"),
                                                         [1, 1], "rr", [1, 1], enqueue=[-2 ** 31])]))


def echo(d, a):
    return Program(f"echo{d}", "f32", Pipeline([FeedbackLoop(Filter("ADD", [2]), Filter("AMPLIFY", [], [a]), [1, 1],
                                                             "dup", enqueue=[0.0] * d)]))


def test_running_sum(oracle_lib):
    x = inputs.keys_i32(1, 5000)
    assert np.array_equal(oracle_lib.run(running_sum(), x, 5000), np.cumsum(x, dtype=np.int32))


def test_running_max_lag(oracle_lib):
    x = inputs.keys_i32(2, 3000)
    prev = np.concatenate([[np.int32(-2 ** 31)], np.maximum.accumulate(x)[:-1]])
    assert np.array_equal(oracle_lib.run(running_max_lag(), x, 3000), np.minimum(x, prev))


@pytest.mark.parametrize("d,a", [(1, 0.5), (7, -0.75), (64, 0.25)])
def test_echo_is_iir(oracle_lib, d, a):
    n = 4000
    x = inputs.uniform_f32(3 + d, n)
    y = oracle_lib.run(echo(d, a), x, n).astype(np.float64)
    den = np.zeros(d + 1)
    den[0], den[d] = 1.0, -a
    ref = scipy.signal.lfilter([1.0], den, x.astype(np.float64))
    # each step adds at most two roundings of a value bounded by max|y|; the recurrence contracts (|a| < 1)
    bound = 4 * 2.0 ** -24 * np.max(np.abs(ref)) / (1 - abs(a))
    assert np.max(np.abs(y - ref)) <= bound


def test_multirate_body(oracle_lib):
    c = [0.5, -2.0, 0.25]
    prog = Program("mr", "f32", Pipeline([FeedbackLoop(Filter("FIR", [3, 3], c), Filter("IDENTITY"), [2, 1], "dup",
                                                       enqueue=[0.0])]))
    n = 2000
    r = oracle_lib.rates(prog)
    assert r["in_per_iter"] == 2 and r["out_per_iter"] == 1
    assert oracle_lib.in_items(prog, n) == 2 * n
    x = inputs.make_input("f32", 2 * n, 5, variant="smallint")
    y = oracle_lib.run(prog, x, n).astype(np.float64)
    u = c[0] * x[0::2].astype(np.float64) + c[1] * x[1::2]
    ref = scipy.signal.lfilter([1.0], [1.0, -c[2]], u)
    assert np.max(np.abs(y - ref)) <= 8 * 2.0 ** -24 * np.max(np.abs(ref))


def test_loop_rates_and_rejection(oracle_lib):
    r = oracle_lib.rates(running_sum())
    assert r["reps"] == [1, 1, 1, 1]
    # loop = EXPAND(2): 2 items return per firing but the joiner takes 1 -> inconsistent balance equations
    bad = Program("bad", "f32", Pipeline([FeedbackLoop(Filter("ADD", [2]), Filter("EXPAND", [2]), [1, 1], "dup",
                                                       enqueue=[0.0])]))
    with pytest.raises(Exception):
        oracle_lib.rates(bad)


def test_feedback_determinism(oracle_lib):
    prog = Program("mix", "f32", Pipeline([Filter("FIR", [4, 1], [0.5, 0.25, -1.0, 2.0]),
                                           FeedbackLoop(Filter("ADD", [2]), Filter("AMPLIFY", [], [0.5]), [1, 1],
                                                        "dup", enqueue=[0.0] * 5),
                                           Filter("DECIMATE", [2])]))
    n = 1500
    x = inputs.uniform_f32(9, oracle_lib.in_items(prog, n))
    base = oracle_lib.run(prog, x, n).tobytes()
    for chunk in (1, 7, 100000):
        for order in (0, 1):
            assert oracle_lib.run(prog, x, n, chunk=chunk, order_seed=order).tobytes() == base
