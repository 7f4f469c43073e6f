"""Pick the headline metrics of one kernel out of an `ncu --page raw --csv` export (one capture)
and print them as metric,unit,value (the profiles/*_ncu_*.csv summaries)."""
import csv
import sys

KEYS = ["Kernel Name", "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "smsp__issue_active.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_tensor_subpipe_dmma.avg.pct_of_peak_sustained_active",
        "sm__throughput.avg.pct_of_peak_sustained_elapsed", "launch__registers_per_thread", "launch__grid_size",
        "launch__block_size", "launch__shared_mem_per_block_dynamic", "l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum",
        "smsp__inst_executed.sum", "lts__t_sector_hit_rate.pct"]
PREFIX = "smsp__pcsamp_warps_issue_stalled_"


def main(path):
    rows = list(csv.reader(open(path)))
    hdr, units, vals = rows[0], rows[1], rows[2]
    print("metric,unit,value")
    for i, h in enumerate(hdr):
        if h in KEYS or (h.startswith(PREFIX) and not h.endswith("_not_issued")):
            print(f'{h},{units[i]},"{vals[i]}"')


if __name__ == "__main__":
    main(sys.argv[1])
