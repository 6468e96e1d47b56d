"""Config-5 fault campaign (tools/campaign.py) at reduced grids with high rates
so every trial has flips.

* full oracle (256^2 and 512^2): every trial's check_all counts, SpMV counts,
  SpMV output words and scrubbed storage bit-identical to the oracle running
  the same trial on its own encoding;
* the large-grid comparison path (touched codewords only) agrees with the GPU
  too, so the 4096^2 campaign's comparison rule is itself checked here;
* ground-truth classification: with the config-2 schemes every single flip is
  corrected or masked and every same-word double flip is a DUE or masked (no
  silent data corruption); the V-SED / R-SED contrast arm turns same-word
  double flips in vectors and row pointers into SDC (SED detects
  odd-weight errors only)."""
import os
import sys

import pytest

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def campaign():
    sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tools"))
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    import campaign as c
    return c


@pytest.mark.parametrize("grid,rates", [(256, [1e-5, 1e-4]), (512, [3e-5])])
def test_campaign_full_oracle(campaign, grid, rates):
    summary, trials = campaign.run(grid, rates, 2, ["single", "double"], None, arms=("secded", "sed"),
                                   full_oracle=True, verbose=False)
    assert summary["all_match_oracle"], [t for t in trials if not t["oracle_match"]]
    assert summary["all_encodings_match"]
    for t in trials:
        assert t["flips"] > 0
        assert t["masked"] + t["corrected"] + t["due"] + t["sdc"] == t["flips"]
        if t["arm"] == "secded":
            assert t["sdc"] == 0
            if t["kind"] == "single":
                assert t["due"] == 0 and t["uncorrectable"] == 0 and t["corrected"] + t["masked"] == t["flips"]
            else:
                assert t["corrected"] == 0 and t["due"] + t["masked"] == t["flips"]
    s_sed_d = summary["sed_double"]
    assert s_sed_d["sdc"] > 0           # even-weight errors pass SED silently
    assert summary["secded_double"]["sdc"] == 0


def test_campaign_touched_codeword_rule(campaign):
    """The comparison rule the 4096^2 campaign uses (oracle check of touched
    codewords + the clean-SpMV identity for single flips) holds on every trial."""
    summary, trials = campaign.run(256, [1e-4], 3, ["single", "double"], None, arms=("secded", "sed"),
                                   full_oracle=False, verbose=False)
    assert summary["all_match_oracle"], [t for t in trials if not t["oracle_match"]]
