"""GPU parity of the NEXT-3 / NEXT-4 layout scan (§5.3: SUM(col1 + ... + colN) over DSM,
PAX and NSM) through the C ABI, from HBM and zero-copy from pinned host memory, against the CPU
oracle (pinned in tests/test_oracle_layout.py) — bit-exact int64 sums."""
import numpy as np
import pytest

import chgen
import oracle

pytestmark = pytest.mark.gpu
LAYOUTS = {"dsm": 1, "pax": 2, "nsm": 3}


@pytest.fixture(scope="module")
def h():
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    return mod


@pytest.fixture(scope="module")
def e(h):
    eng = h.h2tap_open(0)
    yield eng
    h.h2tap_close(eng)


def place(arr, where):
    import torch
    t = torch.from_numpy(np.ascontiguousarray(arr))
    if where == "hbm":
        return t.cuda()
    p = torch.empty(t.shape, dtype=t.dtype, pin_memory=True)
    p.copy_(t)
    return p


@pytest.mark.parametrize("where", ["hbm", "host"])
@pytest.mark.parametrize("n", [1, 3, 64, 65, 4099, 100_003])
def test_parity_small(h, e, where, n):
    m = chgen.layout_matrix(n, 16, seed=n)
    rng = np.random.default_rng(n)
    masks = [[0], [0, 1], list(range(4)), list(range(8)), list(range(16)), [15], sorted(rng.choice(16, 5, replace=False))]
    for lay, lid in LAYOUTS.items():
        data = chgen.encode_layout(m, lay)
        d = place(data, where)
        for cols in masks:
            got, ms = h.h2tap_layout_sum(e, d, lid, n, 16, cols)
            assert got == oracle.layout_sum(data, lay, n, 16, cols), (lay, cols)
            assert ms >= 0


def test_geometries(h, e):
    """DSM with padded column starts, PAX with 16-row minipages, 64-attribute and 4-attribute records."""
    n = 5003
    m16 = chgen.layout_matrix(n, 16, seed=3)
    data = chgen.encode_layout(m16, "dsm", col_stride=n + 5)
    got, _ = h.h2tap_layout_sum(e, place(data, "hbm"), 1, n, 16, [2, 9], col_stride=n + 5)
    assert got == oracle.layout_sum(data, "dsm", n, 16, [2, 9], col_stride=n + 5)
    import torch
    buf = torch.zeros(len(data) + 4, dtype=torch.int32, device="cuda")  # DSM from a 4-byte offset
    buf[1:1 + len(data)] = torch.from_numpy(data).cuda()
    got, _ = h.h2tap_layout_sum(e, buf[1:], 1, n, 16, [0, 3, 15], col_stride=n + 5)
    assert got == oracle.layout_sum(data, "dsm", n, 16, [0, 3, 15], col_stride=n + 5)
    for mp in (16, 256):
        data = chgen.encode_layout(m16, "pax", pax_rows=mp)
        got, _ = h.h2tap_layout_sum(e, place(data, "hbm"), 2, n, 16, [1, 2, 7], pax_rows=mp)
        assert got == oracle.layout_sum(data, "pax", n, 16, [1, 2, 7], pax_rows=mp)
    data = chgen.encode_layout(m16, "pax", pax_rows=16)
    got, _ = h.h2tap_layout_sum(e, place(data, "hbm"), 2, n, 16, [0, 15], pax_rows=16)
    assert got == oracle.layout_sum(data, "pax", n, 16, [0, 15], pax_rows=16)
    for k, cols in ((64, [0, 31, 63]), (4, [1, 3])):
        m = chgen.layout_matrix(n, k, seed=k)
        for lay, lid in LAYOUTS.items():
            data = chgen.encode_layout(m, lay)
            got, _ = h.h2tap_layout_sum(e, place(data, "hbm"), lid, n, k, cols)
            assert got == oracle.layout_sum(data, lay, n, k, cols), (k, lay)


def test_empty_and_errors(h, e):
    import torch
    z = torch.zeros(16, dtype=torch.int32, device="cuda")
    assert h.h2tap_layout_sum(e, z, 1, 0, 16, [0])[0] is None
    for bad in (dict(layout=4, ncols=16, cols=[0]), dict(layout=3, ncols=12, cols=[0]),
                dict(layout=1, ncols=16, cols=[]), dict(layout=1, ncols=16, cols=[16])):
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_layout_sum(e, z, bad["layout"], 4, bad["ncols"], bad["cols"])
        assert ei.value.status == h.H2TAP_EINVAL
    pageable = torch.zeros(64, dtype=torch.int32)
    with pytest.raises(h.H2tapError) as ei:
        h.h2tap_layout_sum(e, pageable, 3, 4, 16, [0])
    assert ei.value.status == h.H2TAP_EINVAL
    with pytest.raises(h.H2tapError) as ei:  # misaligned
        h.h2tap_layout_sum(e, torch.zeros(80, dtype=torch.int32, device="cuda")[1:], 3, 4, 16, [0])
    assert ei.value.status == h.H2TAP_EINVAL


def closed_form(n, k, cols, K):
    """value(r, c) = (r mod K) * k + c: SUM = |S| * k * sum_r (r mod K) + n * sum(S)."""
    q, rem = divmod(n, K)
    s_r = q * K * (K - 1) // 2 + rem * (rem - 1) // 2
    return len(cols) * k * s_r + n * sum(cols)


def build_closed_form(n, k, K, lay, pax_rows=64):
    """The closed-form table built on the device by torch (input construction only)."""
    import torch
    r = (torch.arange(n, device="cuda", dtype=torch.int64) % K).to(torch.int32)
    m = r[:, None] * k + torch.arange(k, device="cuda", dtype=torch.int32)[None, :]
    if lay == "nsm":
        return m.reshape(-1)
    if lay == "dsm":
        return m.t().contiguous().reshape(-1)
    pages = -(-n // pax_rows)
    pad = torch.zeros(pages * pax_rows, k, dtype=torch.int32, device="cuda")
    pad[:n] = m
    return pad.reshape(pages, pax_rows, k).permute(0, 2, 1).contiguous().reshape(-1)


def test_full_size_paper_table(h, e):
    """The paper's 270 M-record x 16-attribute table (≈17 GB, Fig. 10), HBM-resident on one B200
    (the paper had to shrink it to 1 GB for GPU residency, L1031-1034), every layout, N = 1..16."""
    import torch
    n, k, K = 270_000_000, 16, 1 << 20
    for lay, lid in LAYOUTS.items():
        d = build_closed_form(n, k, K, lay)
        for cols in ([0], [0, 1], list(range(4)), list(range(8)), list(range(16))):
            assert h.h2tap_layout_sum(e, d, lid, n, k, cols)[0] == closed_form(n, k, cols, K), (lay, cols)
        del d
        torch.cuda.empty_cache()


def test_host_resident_zero_copy_large(h, e):
    """1 GB pinned host table read over PCIe by the kernel (no copy), every layout."""
    import torch
    n, k, K = 16_777_219, 16, 1 << 16
    for lay, lid in LAYOUTS.items():
        dev = build_closed_form(n, k, K, lay)
        host = torch.empty(dev.shape, dtype=torch.int32, pin_memory=True)
        host.copy_(dev)
        del dev
        for cols in ([0, 1], list(range(16))):
            assert h.h2tap_layout_sum(e, host, lid, n, k, cols)[0] == closed_form(n, k, cols, K), (lay, cols)
