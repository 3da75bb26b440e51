"""GPU parity of the one-pass query over a bit-packed residual (k > 8, BASELINE configs[2] at M = 8 / 12 / 16):
the gathered-residual kernel sends the non-definite candidates to its result ring as check entries
(Alg. 2, on those rows only): the check code -- the candidate's bucket is the one holding
lo and / or the one holding hi -- comes from the definite-range borrow chains, the pass gathers the row's
residual bits with the aggregate, the drain tests them against the low bits of the exact bounds.  COUNT
(check entries only) and SUM through the ring, bounds that exercise every code: unaligned, bucket-aligned,
lo and hi in one bucket, adjacent buckets (no definite bucket), the first and last bucket, the whole domain."""
import numpy as np
import pytest

import datagen
import oracle

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


def _bounds(k):
    b = 1 << k
    return [
        (0x5A5A5A37, 0x5A5A5A37 + (1 << 32) // 10000),      # C3 at 0.01 %, unaligned
        (0x5A5A5A37, 0x5A5A5A37 + (1 << 32) // 100),        # 1 %
        (3 * b, 7 * b - 1),                                 # bucket-aligned: no check entries
        (3 * b + 5, 3 * b + 9),                             # lo and hi in one bucket (code 3)
        (3 * b + 5, 4 * b + 9),                             # adjacent buckets, no definite bucket
        (0, 77),                                            # first bucket only (clo = chi = 0)
        ((1 << 32) - 1 - 77, (1 << 32) - 1),                # last bucket only
        (0, (1 << 32) - 1),                                 # every row
        (12345, 12345),                                     # a point
    ]


@pytest.mark.parametrize("major_bits,loc", [(8, 0), (12, 0), (16, 0), (8, 1), (16, 1)])
def test_gpu_packed_check_entries(cu, major_bits, loc):
    from paper_conf_icde_pirkmk14_b200 import _ar
    k = 32 - major_bits
    n = 5 * 8192 + 3333
    v = datagen.uniform_u32(100 + major_bits, n)
    agg = datagen.uniform_u32(200 + major_bits, n, hi=(1 << 24) - 1)
    # plant rows at the bucket edges the bounds below test (the data must reach the first / last bucket)
    v[:40] = np.arange(40, dtype=np.uint32) * 3
    v[40:80] = (np.uint64(2**32 - 1) - np.arange(40, dtype=np.uint64) * 3).astype(np.uint32)
    col = cu.BWDColumn(v, major_bits, residual_loc=loc)   # loc 1: the residual read over the host link
    assert col.desc.k == k and col.desc.w_major == major_bits
    ag = cu.BWDColumn(agg, 32, layout=_ar.AR_LAYOUT_PACKED)
    for lo, hi in _bounds(k):
        preds = [(col, lo, hi)]
        _, cnt, sm = oracle.select_sum([v], [lo], [hi], [agg], positions=False)
        cpos, cdef = oracle.approx_select([v], [k], [lo], [hi])
        for aggs, want in (([], 0), ([ag], sm)):
            o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
            cu.select_refine_sum(preds, aggs, o4)
            torch.cuda.synchronize()
            assert _ar.ar_last_scan_kernel() == "fused_rg_kernel", (lo, hi)
            assert o4.cpu().tolist() == [want, cnt, cpos.size, int(cdef.sum())], (major_bits, lo, hi, len(aggs))


def test_gpu_packed_check_workspace_pdl(cu):
    """The one-launch form (workspace finalize, programmatic dependent launches) back to back."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 1_000_003
    v = datagen.uniform_u32(7, n)
    agg = datagen.uniform_u32(8, n, hi=(1 << 20) - 1)
    col = cu.BWDColumn(v, 8)
    ag = cu.BWDColumn(agg, 32, layout=_ar.AR_LAYOUT_PACKED)
    lo, hi = 0x12345678, 0x12345678 + (1 << 32) // 200
    _, cnt, sm = oracle.select_sum([v], [lo], [hi], [agg], positions=False)
    cpos, cdef = oracle.approx_select([v], [24], [lo], [hi])
    ws = cu.SrsWorkspace()
    outs = [torch.zeros(4, dtype=torch.int64, device="cuda") for _ in range(4)]
    for o in outs:
        cu.select_refine_sum([(col, lo, hi)], [ag], o, ws=ws, flags=_ar.AR_SRS_PDL_EARLY_READ)
    torch.cuda.synchronize()
    for o in outs:
        assert o.cpu().tolist() == [sm, cnt, cpos.size, int(cdef.sum())]
