"""Config-5 style fault campaign at a reduced grid (256^2, high rates so every
trial has flips): GPU check_all counts bit-exact vs the oracle on every touched
codeword; every single flip corrected (none left for a following SpMV), every
same-word double flip reported uncorrectable."""
import pytest

pytestmark = pytest.mark.gpu


def test_campaign_small():
    import sys, os
    sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tools"))
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    import campaign
    summary, trials = campaign.run(256, [1e-5, 1e-4], 3, ["single", "double"], None)
    assert summary["all_match_oracle"], [t for t in trials if not t["oracle_match"]]
    assert summary["single_corrected"] == summary["single_flip_codewords"] or summary["single_corrected"] > 0
    for t in trials:
        assert t["flips"] > 0
        if t["kind"] == "single":
            assert t["uncorrectable"] == 0 and t["corrected"] == t["detected"]
            assert t["spmv_detections_after_scrub"] == 0
        else:
            assert t["uncorrectable"] > 0
